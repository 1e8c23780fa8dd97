mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_hashjoin_gpu.py -x -q > gpurun_out/pt_k3b.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_k3b.log
for i in 1 2; do
HX_LIB=$PWD/tools/variants/libhx_HF3.so timeout 300 python tools/hashpack_bench.py --sf 100 --parts 8 --reps 5 --no-join 2>&1 | head -3
timeout 300 python tools/hashpack_bench.py --sf 100 --parts 8 --reps 5 --no-join 2>&1 | head -3
done
timeout 300 ncu --clock-control none -k regex:"k3_" -c 6 --csv --metrics gpu__time_duration.sum,dram__bytes_read.sum,smsp__issue_active.avg.pct_of_peak_sustained_active python tools/hashpack_bench.py --sf 100 --parts 8 --reps 2 --no-join > gpurun_out/k3b_ncu.csv 2>&1
grep -v "^==" gpurun_out/k3b_ncu.csv | tail -20
