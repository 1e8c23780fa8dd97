# Builds every native artefact in-tree (the .so files travel to the GPU box with gpurun).
#   ssbgen/libssbgen.so        host input generator          (gcc)
#   ssbgen/libssbgen_cuda.so   device input generator        (nvcc, sm_100a)
#   oracle/liboracle.so        CPU oracle (test infra only)  (g++)
#   paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so   the product C-ABI library (nvcc, sm_100a)
NVCC   ?= /usr/local/cuda/bin/nvcc
ARCH   := -gencode arch=compute_100a,code=sm_100a
PKG    := paper_journals_pvldb_chrysogeloskaa19_b200
NCCL_INC ?= /usr/include
NCCL_LIB ?= $(shell python -c "import nvidia.nccl,os;print(os.path.join(list(nvidia.nccl.__path__)[0],'lib'))" 2>/dev/null)
NVFLAGS := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC -Xcompiler -Wall --expt-relaxed-constexpr

HX_SRC := $(wildcard $(PKG)/csrc/*.cu) $(wildcard $(PKG)/csrc/*.cpp)
HX_HDR := $(wildcard $(PKG)/csrc/*.cuh) $(wildcard $(PKG)/csrc/*.h) include/hx.h

all: ssbgen/libssbgen.so ssbgen/libssbgen_cuda.so oracle/liboracle.so $(if $(wildcard $(PKG)/csrc/*.cu),$(PKG)/libhx.so)

ssbgen/libssbgen.so: ssbgen/ssbgen_host.c ssbgen/ssbgen.h
	gcc -O2 -fopenmp -shared -fPIC -Wall -o $@ ssbgen/ssbgen_host.c

# -Xptxas -O1: ptxas 12.9 -O3 miscompiles two inlined splitmix64 chains in one expression for
# sm_100a (wrong values, reproduced by tools/dbg_gen.cu); -O1 is exact (tests compare every
# device-generated column with the host fill)
ssbgen/libssbgen_cuda.so: ssbgen/ssbgen_cuda.cu ssbgen/ssbgen.h
	$(NVCC) $(NVFLAGS) -Xptxas -O1 -shared -o $@ ssbgen/ssbgen_cuda.cu

oracle/liboracle.so: oracle/ssb_oracle.cpp
	g++ -O2 -std=c++17 -shared -fPIC -Wall -o $@ oracle/ssb_oracle.cpp

$(PKG)/libhx.so: $(HX_SRC) $(HX_HDR)
	$(NVCC) $(NVFLAGS) -Xptxas -v -Iinclude -I$(NCCL_INC) -shared -o $@ $(HX_SRC) \
	  -L$(NCCL_LIB) -l:libnccl.so.2 -Xlinker -rpath=$(NCCL_LIB) 2> $(PKG)/ptxas.log || (cat $(PKG)/ptxas.log; false)

clean:
	rm -f ssbgen/*.so oracle/*.so $(PKG)/*.so

.PHONY: all clean
