mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_R.so tools/variants/libhx_R3.so tools/variants/libhx_SC.so > gpurun_out/ab32.txt 2>&1
bash tools/ab_env.sh 100 "HX_STATIC_CHUNKS=1" "HX_STATIC_CHUNKS=0" >> gpurun_out/ab32.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_R.so tools/variants/libhx_R3.so >> gpurun_out/ab32.txt 2>&1
timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or tiny or ragged or plans_and_graph or segments" > gpurun_out/pt_r3.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_r3.log
