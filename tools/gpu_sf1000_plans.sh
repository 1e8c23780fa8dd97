mkdir -p gpurun_out
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q2.1,q3.1,q4.1,q4.2 > gpurun_out/plans_sf1000.log 2>&1
for e in "HX_K1_W=26" "HX_K1_SMEM_KB=227" "HX_K1_COST=8,120,8,40,40" "HX_K1_COST=8,120,8,20,20"; do echo "== $e"; env $e HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q3.1,q4.1 2>&1 | grep -v "warps=20 \|warps=26 " ; done >> gpurun_out/plans_sf1000.log 2>&1
