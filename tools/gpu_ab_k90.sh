# A/B: 3-stage ring cap for 3-column pipelines (K90: tile ring <= 90 KB) vs default (B1): the plans
# it allows (e.g. Q3.1 with the supplier's full map staged)
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_B1.so tools/variants/libhx_K90.so tools/variants/libhx_B1.so tools/variants/libhx_K90.so > gpurun_out/ab_k90.txt 2>&1
for w in 20 26; do HX_K1_W=$w HX_DEBUG=1 HX_LIB=$PWD/tools/variants/libhx_K90.so timeout 300 python tools/time_queries.py --sf 100 --reps 3 --queries q3.1,q2.1,q3.2 2>&1 | grep -v "warps=$((46-w))" ; done > gpurun_out/plans_k90.log
