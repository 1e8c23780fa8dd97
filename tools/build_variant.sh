# Build a tuning variant of libhx with extra -D flags:  bash tools/build_variant.sh NAME -DX=1 ...
# -> tools/variants/libhx_NAME.so (git-ignored; travels to the GPU box with gpurun)
name=$1; shift
PKG=paper_journals_pvldb_chrysogeloskaa19_b200
NCCL_LIB=$(python -c "import nvidia.nccl,os;print(os.path.join(list(nvidia.nccl.__path__)[0],'lib'))")
mkdir -p tools/variants
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC \
  --expt-relaxed-constexpr -Iinclude -shared "$@" -o tools/variants/libhx_$name.so $PKG/csrc/*.cu \
  -L$NCCL_LIB -l:libnccl.so.2 -Xlinker -rpath=$NCCL_LIB 2>&1 | grep -v "warning #128\|Remark\|^$" | grep -i "error" ; true
