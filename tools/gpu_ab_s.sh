# A/B: slot-tag spin (B0) vs 32 ns sleep between polls (S32), SF100, direct maps and hash tables
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_B0.so tools/variants/libhx_S32.so tools/variants/libhx_B0.so tools/variants/libhx_S32.so > gpurun_out/ab_s.txt 2>&1
JOIN=hash bash tools/ab_libs.sh 100 tools/variants/libhx_B0.so tools/variants/libhx_S32.so tools/variants/libhx_B0.so tools/variants/libhx_S32.so > gpurun_out/ab_s_ht.txt 2>&1
