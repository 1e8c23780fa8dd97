# refresh after the hash-table plan changes: GPU tests, default bench line, SF10 line, smoke
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"
timeout 900 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err; echo "bench rc=$?"
timeout 600 python bench.py --sf 10 --steps 20 --warmup 5 > gpurun_out/bench_sf10.json 2> gpurun_out/bench_sf10.err; echo "sf10 rc=$?"
