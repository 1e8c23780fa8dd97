# A/B (hash-table plans SF100 / SF10): the HT instances' larger warp count 26 (72 registers) vs 24 (80)
mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_V26.so tools/variants/libhx_V24.so tools/variants/libhx_V26.so tools/variants/libhx_V24.so > gpurun_out/ab_v.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_V26.so tools/variants/libhx_V24.so >> gpurun_out/ab_v.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_V24.so timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "instances or in_place" > gpurun_out/pt_v24.log 2>&1; tail -1 gpurun_out/pt_v24.log
