mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_HF4.so tools/variants/libhx_FALL.so tools/variants/libhx_HF4.so tools/variants/libhx_FALL.so > gpurun_out/ab39.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_HF4.so tools/variants/libhx_FALL.so >> gpurun_out/ab39.txt 2>&1
