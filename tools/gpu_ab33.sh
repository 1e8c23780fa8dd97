mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_DYN.so tools/variants/libhx_SC.so > gpurun_out/ab33.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_DYN.so tools/variants/libhx_SC.so >> gpurun_out/ab33.txt 2>&1
bash tools/ab_libs.sh 1 tools/variants/libhx_DYN.so tools/variants/libhx_SC.so >> gpurun_out/ab33.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pt_sc.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_sc.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke(); print('SMOKE OK')" > gpurun_out/smoke_sc.log 2>&1; tail -1 gpurun_out/smoke_sc.log
timeout 900 python bench.py > gpurun_out/bench_sc.json 2> gpurun_out/bench_sc.err; echo "bench rc=$?"
