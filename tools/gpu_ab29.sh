mkdir -p gpurun_out
HX_LIB=$PWD/tools/variants/libhx_R.so bash tools/ab_env.sh 100 "HX_NO_DM=1" > gpurun_out/ab29.txt 2>&1
bash tools/ab_env.sh 100 "HX_NO_DM=1" "HX_X=1" >> gpurun_out/ab29.txt 2>&1
HX_LIB=$PWD/tools/variants/libhx_R.so bash tools/ab_env.sh 10 "HX_NO_DM=1" >> gpurun_out/ab29.txt 2>&1
bash tools/ab_env.sh 10 "HX_NO_DM=1" >> gpurun_out/ab29.txt 2>&1
