# Final r02 refresh of the legs the last plan change touched: SF1000 phases, ncu launch list,
# ncu --set full of the 13 SF100 K1 launches (+ source views of Q2.1/Q3.1/Q4.1)
mkdir -p gpurun_out
for ph in q1.1,q1.2,q1.3 q2.1,q2.2,q2.3,q3.1,q3.2,q3.3,q3.4,q4.1,q4.2,q4.3; do timeout 1200 python bench.py --sf 1000 --queries $ph --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-ht-path > "gpurun_out/bench_sf1000_${ph%%,*}.json" 2> "gpurun_out/bench_sf1000_${ph%%,*}.err"; echo "sf1000 $ph rc=$?"; done
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-ht-path > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:"k1_(probe|scan)_agg" -s 13 -c 13 -o /tmp/k1_full python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/ncu_full.log 2>&1; echo "ncu2 rc=$?"
ncu -i /tmp/k1_full.ncu-rep --page raw --csv > gpurun_out/k1_full_raw.csv 2>/dev/null
for i in 3 6 10; do python tools/ncu_lines.py /tmp/k1_full.ncu-rep --launch $i --rows 6e8 --top 40 > gpurun_out/k1_lines_$i.txt 2>&1; done
