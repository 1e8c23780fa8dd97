# A/B: HEAD (R) vs reciprocal ring-slot division (M), SF100, direct maps and hash tables; ncu source view of M
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_R.so tools/variants/libhx_M.so tools/variants/libhx_R.so tools/variants/libhx_M.so > gpurun_out/ab_m.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_R.so tools/variants/libhx_M.so > gpurun_out/ab_m_ht.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_M.so HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 1 > gpurun_out/plans_m.log 2>&1
HX_LIB=$PWD/tools/variants/libhx_M.so bash tools/gpu_ncu_q.sh 100 q2.1,q3.1,q4.1 /tmp/k1_q
for i in 0 1 2; do python tools/ncu_lines.py /tmp/k1_q.ncu-rep --launch $i --rows 6e8 --top 60 > gpurun_out/k1_lines_m_$i.txt 2>&1; done
ncu -i /tmp/k1_q.ncu-rep --page raw --csv > gpurun_out/k1_q_raw.csv 2>/dev/null
