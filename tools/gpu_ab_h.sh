# A/B: hash-table plans with the most selective unfiltered join probed in place by stage B
# after the stage-F Bloom filter (HX_HT_INPLACE 0 / 1 / 2, build H2), SF100 and SF10; parity
mkdir -p gpurun_out
export HX_LIB=$PWD/tools/variants/libhx_H2.so
HX_HT_INPLACE=2 timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "instances or key_encodings or probe_order or plans or parity_small" > gpurun_out/pt_h2.log 2>&1; echo "pytest rc=$?"; tail -1 gpurun_out/pt_h2.log
JOIN=hash bash tools/ab_env.sh 100 "HX_HT_INPLACE=0" "HX_HT_INPLACE=1" "HX_HT_INPLACE=2" "HX_HT_INPLACE=0" "HX_HT_INPLACE=1" "HX_HT_INPLACE=2" > gpurun_out/ab_h.txt 2>&1
JOIN=hash bash tools/ab_env.sh 10 "HX_HT_INPLACE=0" "HX_HT_INPLACE=2" >> gpurun_out/ab_h.txt 2>&1
HX_HT_INPLACE=2 HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 100 --reps 1 --join hash 2>&1 | grep -v "warps=20" | grep "\[hx\]" > gpurun_out/plans_h.log
