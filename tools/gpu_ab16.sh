mkdir -p gpurun_out
for e in "HX_L2_PERSIST_MB=0" "HX_X=1" "HX_LIB=$PWD/tools/variants/libhx_r01.so"; do
  echo "== $e"; env $e timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 2>&1 | tail -1
done > gpurun_out/ab16.txt 2>&1
bash tools/ab_env.sh 100 "HX_L2_PERSIST_MB=0" "HX_X=1" >> gpurun_out/ab16.txt 2>&1
