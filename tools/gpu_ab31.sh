mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_R.so tools/variants/libhx_R2.so tools/variants/libhx_SC.so > gpurun_out/ab31.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_R2.so tools/variants/libhx_SC.so >> gpurun_out/ab31.txt 2>&1
