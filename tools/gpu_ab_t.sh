# A/B: 2560-row tiles (M2) vs 1280-row tiles with a ring of the same bytes (T1280), SF100
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_M.so tools/variants/libhx_M2.so tools/variants/libhx_T1280.so tools/variants/libhx_M2.so tools/variants/libhx_T1280.so > gpurun_out/ab_t.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_M2.so tools/variants/libhx_T1280.so > gpurun_out/ab_t_ht.txt 2>&1
HX_DEBUG=1 HX_LIB=$PWD/tools/variants/libhx_T1280.so timeout 300 python tools/time_queries.py --sf 100 --reps 1 2>&1 | grep "warps=26" > gpurun_out/plans_t.log
