mkdir -p gpurun_out
HX_LIB=$PWD/tools/variants/libhx_B4.so timeout 900 python -m pytest tests/test_hx_gpu.py tests/test_hashjoin_gpu.py tests/test_nccl_gpu.py -x -q > gpurun_out/pt_b4.log 2>&1; echo "pytest B4 rc=$?"; tail -1 gpurun_out/pt_b4.log
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_K3V.so tools/variants/libhx_B4.so tools/variants/libhx_B4L2.so tools/variants/libhx_K3V.so tools/variants/libhx_B4.so > gpurun_out/ab41.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_K3V.so tools/variants/libhx_B4.so tools/variants/libhx_B4L2.so >> gpurun_out/ab41.txt 2>&1
