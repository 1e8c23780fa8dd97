mkdir -p gpurun_out
for lib in H0 H1 H2 H3; do echo "== $lib"; HX_NO_DM=1 HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 100 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done > gpurun_out/ab17.txt 2>&1
HX_NO_DM=1 HX_DEBUG=1 HX_LIB=$PWD/tools/variants/libhx_H1.so timeout 600 python tools/time_queries.py --sf 100 --reps 1 --queries q4.1,q4.2,q3.1,q2.1 > gpurun_out/ab17_plans.txt 2>&1
