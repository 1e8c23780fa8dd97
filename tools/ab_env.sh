# Same-box A/B of one libhx build under several environment settings:
#   bash tools/ab_env.sh SF "ENV1=a ENV2=b" "ENV1=c" ...
sf=$1; shift
for e in "$@"; do
  echo "== $e"
  env $e timeout 600 python tools/time_queries.py --sf $sf --reps 5 --join ${JOIN:-auto} 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'
done
