# A/B (SF100 and SF10, hash tables and direct maps): HEAD vs W1 (80-register 20-warp HT instances, warp rule)
mkdir -p gpurun_out
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_L0.so tools/variants/libhx_W1.so tools/variants/libhx_L0.so tools/variants/libhx_W1.so > gpurun_out/ab_w.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 10 tools/variants/libhx_L0.so tools/variants/libhx_W1.so >> gpurun_out/ab_w.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_L0.so tools/variants/libhx_W1.so >> gpurun_out/ab_w.txt 2>&1
