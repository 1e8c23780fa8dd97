mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_H4.so tools/variants/libhx_N2.so tools/variants/libhx_N1.so > gpurun_out/ab26.txt 2>&1
