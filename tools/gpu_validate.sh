# Full validation: GPU test suite, smoke, SF1000 against the full oracle (6e9 rows).
set -x
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"; tail -2 gpurun_out/smoke.log
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_gpu.log
HX_TEST_SF1000_FULL=1 timeout 2400 python -m pytest tests/test_sf1000_gpu.py -q -s > gpurun_out/sf1000_full.log 2>&1; echo "sf1000 full rc=$?"; tail -5 gpurun_out/sf1000_full.log
