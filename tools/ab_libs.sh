# Same-box A/B of libhx builds: per-query K1 median at SF (time_queries.py) for each build.
#   bash tools/ab_libs.sh SF lib1.so lib2.so ...   (paths relative to the repo root)
#   JOIN=hash bash tools/ab_libs.sh ...     (plans under HX_JOIN_HASH)
sf=$1; shift
for lib in "$@"; do
  echo "== $lib"
  HX_LIB=$PWD/$lib timeout 600 python tools/time_queries.py --sf $sf --reps 5 --join ${JOIN:-auto} 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
done
