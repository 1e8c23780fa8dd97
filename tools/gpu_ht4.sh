mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_HF.so tools/variants/libhx_PH.so tools/variants/libhx_PHG.so > gpurun_out/ab36.txt 2>&1
JOIN=hash bash tools/ab_env.sh 100 "HX_L2_PERSIST=1" "HX_L2_PERSIST=0" >> gpurun_out/ab36.txt 2>&1
