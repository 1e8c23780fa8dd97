mkdir -p gpurun_out
for lib in H0 H4; do echo "== $lib"; HX_NO_DM=1 HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 100 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab18.txt 2>&1
for lib in H0 H4; do echo "== $lib sf10"; HX_NO_DM=1 HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 10 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done >> gpurun_out/ab18.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_H0.so tools/variants/libhx_H4.so >> gpurun_out/ab18.txt 2>&1
timeout 900 python -m pytest tests/test_hx_gpu.py tests/test_nccl_gpu.py tests/test_hashjoin_gpu.py -x -q > gpurun_out/pt_h4.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_h4.log
