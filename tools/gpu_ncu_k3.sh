mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k3_" -c 3 -o gpurun_out/k3_full python tools/hashpack_bench.py --sf 100 --parts 8 --reps 1 > gpurun_out/k3_ncu.log 2>&1; echo "ncu rc=$?"
