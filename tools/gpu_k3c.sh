mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_hashjoin_gpu.py -x -q > gpurun_out/pt_k3c.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_k3c.log
for i in 1 2; do for v in HF3 K3V K3P; do
echo $v; HX_LIB=$PWD/tools/variants/libhx_$v.so timeout 300 python tools/hashpack_bench.py --sf 100 --parts 8 --reps 5 --no-join 2>&1 | tail -1
done; done
for v in HF3 K3V K3P; do
HX_LIB=$PWD/tools/variants/libhx_$v.so timeout 300 ncu --clock-control none -k regex:"k3_count" -c 2 --csv --metrics gpu__time_duration.sum,smsp__issue_active.avg.pct_of_peak_sustained_active python tools/hashpack_bench.py --sf 100 --parts 8 --reps 2 --no-join 2>&1 | grep k3_count | awk -F'","' -v v=$v '{print v, $13, $15}'
done
