# SF1000 on one GPU (configs[3] 1-GPU baseline, two column phases), host-resident SF100, the
# micro-benchmarks, K3 hash-pack.
set -x
mkdir -p gpurun_out
for ph in q1.1,q1.2,q1.3 q2.1,q2.2,q2.3,q3.1,q3.2,q3.3,q3.4,q4.1,q4.2,q4.3; do timeout 1200 python bench.py --sf 1000 --queries $ph --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-ht-path > "gpurun_out/bench_sf1000_${ph%%,*}.json" 2> "gpurun_out/bench_sf1000_${ph%%,*}.err"; echo "sf1000 $ph rc=$?"; done
for w in sum join; do timeout 600 python bench.py --workload $w --steps 10 > gpurun_out/bench_$w.json 2> gpurun_out/bench_$w.err; echo "$w rc=$?"; done
timeout 600 python bench.py --variant host --sf 100 --steps 3 --warmup 1 --no-cpu-baseline > gpurun_out/bench_host_sf100.json 2> gpurun_out/bench_host_sf100.err; echo "host100 rc=$?"
timeout 600 python bench.py --variant uva --steps 5 --sf 10 --no-cpu-baseline > gpurun_out/bench_uva.json 2> gpurun_out/bench_uva.err; echo "uva rc=$?"
timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 > gpurun_out/hashpack.jsonl 2> gpurun_out/hashpack.err; echo "hashpack rc=$?"
timeout 600 python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err; echo "ref rc=$?"
