mkdir -p gpurun_out
for lib in H4 K1 K2 K3 H4; do echo "== $lib"; HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 2>&1 | tail -1; done > gpurun_out/ab19.txt 2>&1
