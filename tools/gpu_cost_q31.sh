# Q2.1/Q3.1/Q4.1 plans and K1 times at SF100 under several cost-model constants (plan exploration)
mkdir -p gpurun_out
for c in "8,60,8,20,40" "8,60,8,40,40" "8,60,8,10,40" "8,60,8,20,80" "8,60,8,20,20" "8,30,8,20,40" "8,120,8,20,40" "4,60,8,20,40" "16,60,8,20,40"; do
  echo "== $c"
  HX_K1_W=26 HX_DEBUG=1 HX_K1_COST=$c HX_LIB=$PWD/tools/variants/libhx_M.so timeout 300 python tools/time_queries.py --sf 100 --reps 5 --queries q2.1,q3.1,q4.1,q3.2 2>&1 | grep -v "warps=20"
done > gpurun_out/cost_q31.txt 2>&1
