mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_W24.so tools/variants/libhx_W26.so tools/variants/libhx_W24T1280.so tools/variants/libhx_W24T3840.so tools/variants/libhx_W26T1280.so > gpurun_out/ab10_sf100.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_B2r.so tools/variants/libhx_W24.so tools/variants/libhx_W26.so tools/variants/libhx_W24T1280.so > gpurun_out/ab10_sf10.txt 2>&1
