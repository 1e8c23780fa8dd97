set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_nccl_gpu.py tests/test_multigpu_gpu.py -x -q > gpurun_out/pt_nccl.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pt_nccl.log
timeout 900 python bench.py --workload sum --sizeup --steps 10 --warmup 3 > gpurun_out/sizeup_sum.jsonl 2> gpurun_out/sizeup_sum.err; echo "sum rc=$?"
timeout 900 python bench.py --workload join --sizeup --steps 10 --warmup 3 > gpurun_out/sizeup_join.jsonl 2> gpurun_out/sizeup_join.err; echo "join rc=$?"
timeout 600 python bench.py --sf 1 --queries q1.1 --l2-flush --steps 20 --warmup 5 --no-ht-path > gpurun_out/bench_c1.json 2> gpurun_out/bench_c1.err; echo "c1 rc=$?"
timeout 600 python bench.py --sf 10 --steps 20 --warmup 5 --no-e2e > gpurun_out/bench_sf10.json 2> gpurun_out/bench_sf10.err; echo "sf10 rc=$?"
