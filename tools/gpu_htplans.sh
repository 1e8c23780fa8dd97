mkdir -p gpurun_out
HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 3 --join hash 2>&1 | grep -v "warps=20" > gpurun_out/plans_ht.log
