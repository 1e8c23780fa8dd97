set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or ragged or misaligned or segments or tiny or plans_and_graph or host_resident or empty_fact or reserved" > gpurun_out/pt_quick.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_quick.log
bash tools/ab_libs.sh 100 tools/variants/libhx_r01.so tools/variants/libhx_a.so paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so > gpurun_out/ab_sf100.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_r01.so paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so > gpurun_out/ab_sf10.txt 2>&1
