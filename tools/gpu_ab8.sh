mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_B2.so tools/variants/libhx_B2r.so tools/variants/libhx_R96.so tools/variants/libhx_R72.so > gpurun_out/ab8_sf100.txt 2>&1
