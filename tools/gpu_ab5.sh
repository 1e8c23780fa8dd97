mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "small_sf or ragged or misaligned or segments or tiny or plans_and_graph or host_resident or empty_fact or reserved or full_size" > gpurun_out/pt_quick.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_quick.log
bash tools/ab_libs.sh 100 tools/variants/libhx_r01.so tools/variants/libhx_B2.so > gpurun_out/ab5_sf100.txt 2>&1
for lib in tools/variants/libhx_r01.so tools/variants/libhx_B2.so; do
  echo "== $lib"
  HX_LIB=$PWD/$lib timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
done > gpurun_out/ab5_sf1000.txt 2>&1
