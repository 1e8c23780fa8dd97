mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_narrow_gpu.py -x -q > gpurun_out/pt_nw.log 2>&1; echo "pytest rc=$?"; tail -15 gpurun_out/pt_nw.log
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or tiny or ragged or plans_and_graph or segments or misaligned or host" > gpurun_out/pt_nw2.log 2>&1; echo "pytest2 rc=$?"; tail -2 gpurun_out/pt_nw2.log
