mkdir -p gpurun_out
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q4.1,q4.2,q4.3,q3.1 > gpurun_out/ab4_plans.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_r01.so HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q4.1,q4.2,q4.3,q3.1 > gpurun_out/ab4_plans_r01.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_r01.so tools/variants/libhx_B.so > gpurun_out/ab4_sf10.txt 2>&1
