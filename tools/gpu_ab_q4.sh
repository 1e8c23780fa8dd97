# A/B (hash tables SF100 x2, SF10; direct maps SF100): W1 (before) vs Q4 (4-join rotation on the static 20-warp instance)
mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_W1.so tools/variants/libhx_Q4.so tools/variants/libhx_W1.so tools/variants/libhx_Q4.so > gpurun_out/ab_q4.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_W1.so tools/variants/libhx_Q4.so >> gpurun_out/ab_q4.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_W1.so tools/variants/libhx_Q4.so >> gpurun_out/ab_q4.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_Q4.so timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "instances or in_place or probe_order" > gpurun_out/pt_q4.log 2>&1; tail -1 gpurun_out/pt_q4.log
