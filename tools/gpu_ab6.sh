mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_B2.so tools/variants/libhx_B3.so tools/variants/libhx_B4.so tools/variants/libhx_B5.so tools/variants/libhx_B6.so > gpurun_out/ab6_sf100.txt 2>&1
