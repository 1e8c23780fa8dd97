# A/B (hash-table plans, SF100): 20-warp HT instances capped at 72 registers (L0) vs 80 (L1);
# stage-B rotation also for 4-join plans (HX_HT_INPLACE_MAXJ=4)
mkdir -p gpurun_out
for lib in L0 L1; do
  export HX_LIB=$PWD/tools/variants/libhx_$lib.so
  echo "#### $lib"
  JOIN=hash bash tools/ab_env.sh 100 "HX_K1_W=26" "HX_K1_W=20" "HX_K1_W=20 HX_HT_INPLACE_MAXJ=4" "HX_K1_W=26 HX_HT_INPLACE_MAXJ=4"
done > gpurun_out/ab_l.txt 2>&1
