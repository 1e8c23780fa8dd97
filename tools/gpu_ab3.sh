mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_r01.so tools/variants/libhx_A.so tools/variants/libhx_B.so tools/variants/libhx_C.so tools/variants/libhx_D.so > gpurun_out/ab3_sf100.txt 2>&1
for lib in tools/variants/libhx_r01.so tools/variants/libhx_A.so tools/variants/libhx_D.so; do
  for pm in 0 1000; do
    echo "== $lib persist_mb=$pm"
    HX_LIB=$PWD/$lib HX_L2_PERSIST_MB=$pm timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q2.1,q3.1,q3.2,q4.1,q4.2,q4.3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
  done
done > gpurun_out/ab3_sf1000.txt 2>&1
