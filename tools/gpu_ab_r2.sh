mkdir -p gpurun_out
JOIN=hash bash tools/ab_env.sh 100 "HX_HT_INPLACE=1" "HX_HT_INPLACE=2" "HX_HT_INPLACE=1" "HX_HT_INPLACE=2" > gpurun_out/ab_r2.txt 2>&1
JOIN=hash bash tools/ab_env.sh 10 "HX_HT_INPLACE=1" "HX_HT_INPLACE=2" >> gpurun_out/ab_r2.txt 2>&1
