mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or tiny or plans_and_graph or key_enc or permutation" > gpurun_out/pt_b2.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_b2.log
for e in "HX_NO_BML2=1" "HX_X=1" "HX_K1_COST=8,60,8,20,40,15" "HX_K1_COST=8,60,8,20,40,35"; do echo "== $e"; env $e timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab23.txt 2>&1
bash tools/ab_env.sh 100 "HX_NO_BML2=1" "HX_X=1" >> gpurun_out/ab23.txt 2>&1
HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 1 --queries q3.1,q4.1,q4.2 2>&1 | grep "warps=20" > gpurun_out/ab23_plans.txt
