mkdir -p gpurun_out
bash tools/ab_env.sh 100 "HX_K1_W_TOL=1.02" "HX_K1_W_TOL=1.1" "HX_K1_W_TOL=1.25" "HX_K1_W_TOL=1.5" > gpurun_out/ab13_sf100.txt 2>&1
bash tools/ab_env.sh 10 "HX_K1_W_TOL=1.02" "HX_K1_W_TOL=1.1" "HX_K1_W_TOL=1.25" "HX_K1_W_TOL=1.5" > gpurun_out/ab13_sf10.txt 2>&1
for t in 1.02 1.25; do echo "== tol $t"; HX_K1_W_TOL=$t timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab13_sf1000.txt 2>&1
