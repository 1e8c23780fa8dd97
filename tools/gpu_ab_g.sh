# A/B: R3 (HEAD) vs G (stage-C-only join keys gathered instead of staged), direct maps SF100 x2, SF10, SF1000 dims; parity of G
mkdir -p gpurun_out
HX_LIB=$PWD/tools/variants/libhx_G.so timeout 1200 python -m pytest tests/test_hx_gpu.py tests/test_sf1000_gpu.py -x -q > gpurun_out/pt_g.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_g.log
bash tools/ab_libs.sh 100 tools/variants/libhx_R3.so tools/variants/libhx_G.so tools/variants/libhx_R3.so tools/variants/libhx_G.so > gpurun_out/ab_g.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_R3.so tools/variants/libhx_G.so >> gpurun_out/ab_g.txt 2>&1
for lib in R3 G; do echo "== $lib SF1000 dims"; HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done >> gpurun_out/ab_g.txt
HX_LIB=$PWD/tools/variants/libhx_G.so HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 1 2>&1 | grep "\[hx\]" | grep -v "warps=20" > gpurun_out/plans_g.log
