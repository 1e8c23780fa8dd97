mkdir -p gpurun_out
for lib in H4 H5; do echo "== $lib"; HX_NO_DM=1 HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 100 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab24.txt 2>&1
for lib in H4 H5; do echo "== $lib sf10"; HX_NO_DM=1 HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 10 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done >> gpurun_out/ab24.txt 2>&1
