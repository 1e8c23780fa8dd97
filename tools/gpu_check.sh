# Round-2 check: GPU tests, the default bench line (SF100), K1 per query with / without the
# L2 residency features.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
make -s all
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_gpu.log
timeout 900 python bench.py --steps 20 --warmup 5 > gpurun_out/bench.json 2> gpurun_out/bench.err; echo "bench rc=$?"
HX_L2_HINT=0 HX_L2_PERSIST_MB=0 timeout 600 python tools/time_queries.py --sf 100 --reps 5 > gpurun_out/tq_nol2.txt 2>&1
HX_L2_HINT=1 HX_L2_PERSIST_MB=0 timeout 600 python tools/time_queries.py --sf 100 --reps 5 > gpurun_out/tq_hint.txt 2>&1
timeout 600 python tools/time_queries.py --sf 100 --reps 5 > gpurun_out/tq_l2.txt 2>&1
