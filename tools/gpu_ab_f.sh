# A/B: M2 vs F (in-place plans checked against their own footprint) at SF10 / SF100 / SF1000 dims;
# hash-table plans and ncu source view of the hash-table K1 (Q2.1, Q3.1, Q4.1)
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_M2.so tools/variants/libhx_F.so > gpurun_out/ab_f.txt 2>&1
bash tools/ab_libs.sh 10 tools/variants/libhx_M2.so tools/variants/libhx_F.so tools/variants/libhx_M2.so tools/variants/libhx_F.so >> gpurun_out/ab_f.txt 2>&1
for lib in M2 F; do echo "== $lib SF1000 dims"; HX_LIB=$PWD/tools/variants/libhx_$lib.so timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 2>&1 | awk '{printf "%s %s  ", $1, $6} END {print ""}'; done >> gpurun_out/ab_f.txt
JOIN=hash HX_DEBUG=1 HX_LIB=$PWD/tools/variants/libhx_F.so timeout 300 python tools/time_queries.py --sf 100 --reps 1 2>&1 | grep -v "warps=20" > gpurun_out/plans_ht.log
JOIN=hash HX_LIB=$PWD/tools/variants/libhx_F.so bash tools/gpu_ncu_q.sh 100 q2.1,q3.1,q4.1 /tmp/k1_ht
for i in 0 1 2; do python tools/ncu_lines.py /tmp/k1_ht.ncu-rep --launch $i --rows 6e8 --top 50 > gpurun_out/k1_lines_ht_$i.txt 2>&1; done
