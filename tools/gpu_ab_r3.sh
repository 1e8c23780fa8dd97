mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_Q4.so tools/variants/libhx_R3.so tools/variants/libhx_Q4.so tools/variants/libhx_R3.so > gpurun_out/ab_r3.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_Q4.so tools/variants/libhx_R3.so >> gpurun_out/ab_r3.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_R3.so timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "instances or in_place or probe_order" > gpurun_out/pt_r3.log 2>&1; tail -1 gpurun_out/pt_r3.log
