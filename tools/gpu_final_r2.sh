# Round-2 final measurement pass at HEAD (the .ncu-rep files are summarised on the box: gpurun
# copies back at most 64 MiB).
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"
( time timeout 900 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err ) 2> gpurun_out/bench_time.txt; echo "bench rc=$?"
timeout 600 python bench.py --impl reference > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err; echo "ref rc=$?"
timeout 600 python bench.py --sf 10 --steps 20 --warmup 5 > gpurun_out/bench_sf10.json 2> gpurun_out/bench_sf10.err; echo "sf10 rc=$?"
timeout 600 python bench.py --sf 1 --queries q1.1 --l2-flush --steps 20 --warmup 5 > gpurun_out/bench_c1.json 2> gpurun_out/bench_c1.err; echo "c1 rc=$?"
for w in sum join; do timeout 600 python bench.py --workload $w --steps 10 > gpurun_out/bench_$w.json 2> gpurun_out/bench_$w.err; echo "$w rc=$?"; done
timeout 900 python bench.py --variant host --queries q2.1,q3.1,q4.1 --steps 3 --warmup 1 --no-cpu-baseline > gpurun_out/bench_host_sf100.json 2> gpurun_out/bench_host_sf100.err; echo "host rc=$?"
timeout 600 python bench.py --variant uva --sf 10 --queries q2.1,q3.1,q4.1 --steps 5 --no-cpu-baseline > gpurun_out/bench_uva.json 2> gpurun_out/bench_uva.err; echo "uva rc=$?"
timeout 600 python bench.py --variant host --router shared --sf 10 --queries q2.1,q3.1,q4.1 --steps 3 --warmup 1 --no-cpu-baseline > gpurun_out/bench_host_shared.json 2> gpurun_out/bench_host_shared.err; echo "shared rc=$?"
for ph in q1.1,q1.2,q1.3 q2.1,q2.2,q2.3,q3.1,q3.2,q3.3,q3.4,q4.1,q4.2,q4.3; do timeout 1200 python bench.py --sf 1000 --queries $ph --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-ht-path > "gpurun_out/bench_sf1000_${ph%%,*}.json" 2> "gpurun_out/bench_sf1000_${ph%%,*}.err"; echo "sf1000 $ph rc=$?"; done
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-ht-path > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:"k1_(probe|scan)_agg" -s 13 -c 13 -o /tmp/k1_full python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/ncu_full.log 2>&1; echo "ncu2 rc=$?"
ncu -i /tmp/k1_full.ncu-rep --page raw --csv > gpurun_out/k1_full_raw.csv 2>/dev/null
for i in 3 6 10; do python tools/ncu_lines.py /tmp/k1_full.ncu-rep --launch $i --rows 6e8 --top 40 > gpurun_out/k1_lines_$i.txt 2>&1; done
du -sh gpurun_out
