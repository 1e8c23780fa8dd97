mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_H4.so tools/variants/libhx_R.so > gpurun_out/ab27.txt 2>&1
timeout 900 python -m pytest tests/test_hx_gpu.py tests/test_hashjoin_gpu.py tests/test_nccl_gpu.py -x -q > gpurun_out/pt_r.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_r.log
