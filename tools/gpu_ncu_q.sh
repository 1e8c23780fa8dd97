# ncu --set full of K1 for selected queries at SF (source-level)
sf=${1:-100}; qs=${2:-q2.1,q3.1,q4.1}; out=${3:-gpurun_out/k1_q}
n=$(echo $qs | tr ',' '\n' | wc -l)
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k1_probe_agg" -s $n -c $n -o $out python tools/prof_query.py --sf $sf --queries $qs --reps 2 --join ${JOIN:-auto} > ${out}.log 2>&1; echo "ncu rc=$?"
