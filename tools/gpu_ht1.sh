mkdir -p gpurun_out
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 100 --reps 3 --join hash > gpurun_out/ht_plans.txt 2>&1
JOIN=hash bash tools/gpu_ncu_q.sh 100 q2.1,q3.1,q4.1,q4.2 /tmp/k1_ht
for q in 0 1 2 3; do :; done
ncu -i /tmp/k1_ht.ncu-rep --page raw --csv > gpurun_out/k1_ht_raw.csv 2>/dev/null
ncu -i /tmp/k1_ht.ncu-rep --page source --csv --print-source sass > gpurun_out/k1_ht_src.csv 2>/dev/null
ls -la gpurun_out/k1_ht*
