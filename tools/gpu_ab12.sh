mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or ragged or misaligned or segments or tiny or plans_and_graph or host_resident or empty_fact or reserved or key_enc" > gpurun_out/pt_quick.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_quick.log
HX_K1_W=20 timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or ragged or tiny or plans_and_graph" > gpurun_out/pt_quick20.log 2>&1; echo "pytest20 rc=$?"; tail -2 gpurun_out/pt_quick20.log
HX_K1_W=26 timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or ragged or tiny or plans_and_graph" > gpurun_out/pt_quick26.log 2>&1; echo "pytest26 rc=$?"; tail -2 gpurun_out/pt_quick26.log
bash tools/ab_libs.sh 100 tools/variants/libhx_B2r.so tools/variants/libhx_W26.so tools/variants/libhx_D2.so tools/variants/libhx_D3.so > gpurun_out/ab12_sf100.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_B2r.so tools/variants/libhx_D2.so tools/variants/libhx_D3.so > gpurun_out/ab12_sf10.txt 2>&1
