set -x
mkdir -p gpurun_out
timeout 900 python bench.py --variant host --router shared --sf 10 --steps 3 --warmup 1 > gpurun_out/bench_host_shared.json 2> gpurun_out/bench_host_shared.err; echo "shared rc=$?"
timeout 900 python bench.py --variant host --sf 10 --steps 3 --warmup 1 --no-cpu-baseline > gpurun_out/bench_host_static.json 2> gpurun_out/bench_host_static.err; echo "static rc=$?"
