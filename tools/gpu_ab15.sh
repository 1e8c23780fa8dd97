mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_E1.so tools/variants/libhx_E2.so tools/variants/libhx_E3.so tools/variants/libhx_E4.so tools/variants/libhx_E1.so > gpurun_out/ab15_sf100.txt 2>&1
