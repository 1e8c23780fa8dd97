mkdir -p gpurun_out
HX_LIB=$PWD/tools/variants/libhx_M.so bash tools/ab_env.sh 100 "HX_X=0" "HX_K1_PREFETCH=2" "HX_K1_PREFETCH=4" "HX_K1_W=20" "HX_K1_W=20 HX_K1_PREFETCH=2" "HX_K1_PREFETCH=1" "HX_X=0" > gpurun_out/env_m.txt 2>&1
