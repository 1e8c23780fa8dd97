mkdir -p gpurun_out
timeout 900 python bench.py --encoding narrow --steps 20 --warmup 5 --no-e2e --no-cpu-baseline > gpurun_out/bench_narrow.json 2> gpurun_out/bench_narrow.err; echo "narrow rc=$?"
timeout 900 python bench.py --encoding narrow --sf 10 --steps 20 --warmup 5 --no-e2e --no-cpu-baseline > gpurun_out/bench_narrow_sf10.json 2> gpurun_out/bench_narrow_sf10.err; echo "narrow10 rc=$?"
timeout 900 python bench.py --steps 20 --warmup 5 --no-e2e --no-cpu-baseline > gpurun_out/bench_int32.json 2> gpurun_out/bench_int32.err; echo "int32 rc=$?"
