mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_HF2.so tools/variants/libhx_HTD.so tools/variants/libhx_HF2.so tools/variants/libhx_HTD.so > gpurun_out/ab37.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_HF2.so tools/variants/libhx_HTD.so >> gpurun_out/ab37.txt 2>&1
