# cost-model stage-C entry constant c: all 13 queries at SF100, SF10 and SF1000 dimensions (600 M rows)
mkdir -p gpurun_out
for c in "8,60,8,20,40" "8,90,8,20,40" "8,120,8,20,40" "8,150,8,20,40" "8,60,8,20,40"; do
  echo "== $c SF100"; HX_K1_COST=$c timeout 300 python tools/time_queries.py --sf 100 --reps 5 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
  echo "== $c SF10"; HX_K1_COST=$c timeout 300 python tools/time_queries.py --sf 10 --reps 5 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
  echo "== $c SF1000 dims"; HX_K1_COST=$c timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
done > gpurun_out/ccost.txt 2>&1
