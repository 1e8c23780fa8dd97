mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_B2r.so tools/variants/libhx_R72.so tools/variants/libhx_R64.so tools/variants/libhx_W24.so tools/variants/libhx_W28.so tools/variants/libhx_W16.so > gpurun_out/ab9_sf100.txt 2>&1
