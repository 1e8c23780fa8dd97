mkdir -p gpurun_out
HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 1 --join hash 2>&1 | grep "K1 warps" > gpurun_out/ht9_plans.txt
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_HF4.so tools/variants/libhx_HF5.so > gpurun_out/ab40.txt 2>&1
JOIN=hash bash tools/ab_env.sh 100 "HX_F_ALL_MIN=0" "HX_F_ALL_MIN=0.05" "HX_F_ALL_MIN=0.15" "HX_F_ALL_MIN=99" >> gpurun_out/ab40.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_HF4.so tools/variants/libhx_HF5.so >> gpurun_out/ab40.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_HF4.so tools/variants/libhx_HF5.so >> gpurun_out/ab40.txt 2>&1
