# Round measurement: GPU tests, the default bench line, the micro / host / uva variants,
# the ncu launch list of the bench command and one ncu --set full capture of K1 (13 queries).
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err; echo "bench rc=$?"
for w in sum join; do timeout 600 python bench.py --workload $w --steps 10 > gpurun_out/bench_$w.json 2> gpurun_out/bench_$w.err; echo "$w rc=$?"; done
for v in host uva; do timeout 600 python bench.py --variant $v --steps 5 --no-cpu-baseline > gpurun_out/bench_$v.json 2> gpurun_out/bench_$v.err; echo "$v rc=$?"; done
timeout 600 python bench.py --sf 100 --steps 10 --no-e2e --no-cpu-baseline > gpurun_out/bench_sf100.json 2> gpurun_out/bench_sf100.err; echo "sf100 rc=$?"
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err; echo "ref rc=$?"
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k1_(probe|scan)_agg" -s 13 -c 13 -o gpurun_out/k1_full python tools/prof_query.py --sf 10 --queries all --reps 2 > gpurun_out/ncu_full.log 2>&1; echo "ncu2 rc=$?"
for ph in q1.1,q1.2,q1.3 q2.1,q2.2,q2.3,q3.1,q3.2,q3.3,q3.4,q4.1,q4.2,q4.3; do timeout 900 python bench.py --sf 1000 --queries $ph --steps 5 --warmup 3 --no-e2e --no-cpu-baseline > "gpurun_out/bench_sf1000_${ph%%,*}.json" 2> "gpurun_out/bench_sf1000_${ph%%,*}.err"; echo "sf1000 $ph rc=$?"; done
