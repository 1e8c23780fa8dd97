# hash-table Q4.x (SF100): chunk claims (default) vs static chunks for 4 joins (S4), each with and
# without the stage-B rotation (HX_HT_INPLACE_MAXJ=4), 20 / 26 warps
mkdir -p gpurun_out
for lib in W1 S4; do
  export HX_LIB=$PWD/tools/variants/libhx_$lib.so; echo "#### $lib"
  for e in "HX_K1_W=26" "HX_K1_W=26 HX_HT_INPLACE_MAXJ=4" "HX_K1_W=20" "HX_K1_W=20 HX_HT_INPLACE_MAXJ=4"; do
    echo "== $e"; env $e timeout 300 python tools/time_queries.py --sf 100 --reps 5 --join hash --queries q4.1,q4.2,q4.3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
  done
done > gpurun_out/ab_s4.txt 2>&1
