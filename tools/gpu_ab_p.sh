# A/B: producer poll sleep 128 ns (M2) vs 0 (P0) vs 32 ns (P32), SF100
mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_M2.so tools/variants/libhx_P0.so tools/variants/libhx_P32.so tools/variants/libhx_M2.so tools/variants/libhx_P0.so tools/variants/libhx_P32.so > gpurun_out/ab_p.txt 2>&1
