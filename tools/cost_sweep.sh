# K1 cost-model sweep at SF1000 dims (600 M-row lineorder prefix) and SF10: per-query K1 time
# for each HX_K1_COST setting given as arguments ("s,c,sc,l2,s2,s2b").
mkdir -p gpurun_out
for c in "$@"; do
  echo "COST $c"
  HX_K1_COST=$c HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | grep -v "joins=0" | cut -c1-260
  HX_K1_COST=$c timeout 300 python tools/time_queries.py --sf 10 --reps 5 2>&1 | grep -v "^\[hx\]"
done
