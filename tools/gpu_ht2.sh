mkdir -p gpurun_out
HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 1 --join hash 2>&1 | grep "K1 warps" > gpurun_out/ht2_plans.txt
JOIN=hash bash tools/ab_env.sh 100 "HX_NONE=1" "HX_HT_FIRST_MIN=99" "HX_HT_FIRST_MIN=0" "HX_HT_FIRST_MIN=0.2" "HX_HT_FIRST_MIN=0.05" "HX_HT_FIRST_MIN=99" > gpurun_out/ab34.txt 2>&1
