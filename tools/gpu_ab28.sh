mkdir -p gpurun_out
bash tools/ab_env.sh 100 "HX_NO_DM=1" "HX_NO_DM=1 HX_HT_STAGES=3" "HX_NO_DM=1 HX_HT_STAGES=2" > gpurun_out/ab28.txt 2>&1
bash tools/ab_env.sh 10 "HX_NO_DM=1" "HX_NO_DM=1 HX_HT_STAGES=3" >> gpurun_out/ab28.txt 2>&1
