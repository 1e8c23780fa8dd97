# L2 residency A/B (SF100 and SF1000 dimensions) + the default bench line and launch list.
set -x
mkdir -p gpurun_out
bash tools/ab_env.sh 100 "HX_X=1" "HX_L2_PERSIST=1" "HX_LIB=$PWD/tools/variants/libhx_PH.so" "HX_L2_PERSIST=1 HX_LIB=$PWD/tools/variants/libhx_PH.so" > gpurun_out/l2ab_sf100.txt 2>&1
for e in "HX_X=1" "HX_L2_PERSIST=1" "HX_LIB=$PWD/tools/variants/libhx_PH.so" "HX_L2_PERSIST=1 HX_LIB=$PWD/tools/variants/libhx_PH.so"; do echo "== $e"; env $e timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/l2ab_sf1000.txt 2>&1
timeout 900 python bench.py --steps 20 --warmup 5 > gpurun_out/bench.json 2> gpurun_out/bench.err; echo "bench rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-ht-path > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 > gpurun_out/hashpack.jsonl 2> gpurun_out/hashpack.err; echo "hashpack rc=$?"
