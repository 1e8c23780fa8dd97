# plan exploration with in-place footprints (build F): compaction cost c
mkdir -p gpurun_out
for c in "8,60,8,20,40" "8,200,8,20,40" "8,300,8,20,40" "8,500,8,20,40"; do
  echo "== $c"
  HX_K1_W=26 HX_DEBUG=1 HX_K1_COST=$c HX_LIB=$PWD/tools/variants/libhx_F.so timeout 300 python tools/time_queries.py --sf 100 --reps 5 2>&1 | grep -v "warps=20"
done > gpurun_out/cost3.txt 2>&1
