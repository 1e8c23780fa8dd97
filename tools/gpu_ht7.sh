mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_HF2.so tools/variants/libhx_HF3.so > gpurun_out/ab38.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_HF2.so tools/variants/libhx_HF3.so >> gpurun_out/ab38.txt 2>&1
timeout 900 python -m pytest tests/test_hx_gpu.py tests/test_nccl_gpu.py -x -q > gpurun_out/pt_ht7.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_ht7.log
