mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pytest_gpu.log
JOIN=hash bash tools/ab_env.sh 100 "HX_HT_INPLACE=0" "HX_HT_INPLACE=1" > gpurun_out/ab_h3.txt 2>&1
