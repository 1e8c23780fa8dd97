mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_R.so tools/variants/libhx_F1.so tools/variants/libhx_F2.so tools/variants/libhx_F3.so > gpurun_out/ab30.txt 2>&1
