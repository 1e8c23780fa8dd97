# Exploration pass: K1 plans and per-query times at SF100 (direct maps and hash tables),
# and an ncu source-level capture of the probe-heavy pipelines.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
make -s all
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 100 --reps 5 > gpurun_out/x_dm_sf100.txt 2>&1; echo rc=$?
HX_NO_DM=1 HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 100 --reps 5 > gpurun_out/x_ht_sf100.txt 2>&1; echo rc=$?
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 10 --reps 5 > gpurun_out/x_dm_sf10.txt 2>&1; echo rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k1_probe_agg" -s 3 -c 3 -o gpurun_out/x_k1_sf100 python tools/prof_query.py --sf 100 --queries q2.1,q3.1,q4.1 --reps 2 > gpurun_out/x_ncu.log 2>&1; echo rc=$?
