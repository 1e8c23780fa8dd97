# ncu --set full of the 13 K1 launches of the hash-table plans (the bench's ht_path) at SF100
mkdir -p gpurun_out
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:"k1_probe_agg" -s 13 -c 13 -o /tmp/k1_ht python tools/prof_query.py --sf 100 --queries all --reps 2 --join hash > gpurun_out/ncu_ht.log 2>&1; echo "ncu rc=$?"
ncu -i /tmp/k1_ht.ncu-rep --page raw --csv > gpurun_out/k1_ht_raw.csv 2>/dev/null
for i in 6 10 11; do python tools/ncu_lines.py /tmp/k1_ht.ncu-rep --launch $i --rows 6e8 --top 40 > gpurun_out/k1_ht_lines_$i.txt 2>&1; done
