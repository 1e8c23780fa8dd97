mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or tiny or ragged or plans_and_graph or misaligned or segments" > gpurun_out/pt_p1.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_p1.log
bash tools/ab_libs.sh 100 tools/variants/libhx_P0.so tools/variants/libhx_P1.so tools/variants/libhx_P2.so > gpurun_out/ab20.txt 2>&1
for lib in P0 P1 P2; do echo "== $lib"; HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab20_sf1000.txt 2>&1
