mkdir -p gpurun_out
for w in 20 26; do echo "== W$w"; HX_K1_W=$w HX_DEBUG=1 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q3.1,q4.1,q4.3 2>&1; done > gpurun_out/ab14.txt
echo "== D2 W20" >> gpurun_out/ab14.txt; HX_LIB=$PWD/tools/variants/libhx_D2.so HX_K1_W=20 timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q3.1,q4.1,q4.3 >> gpurun_out/ab14.txt 2>&1
echo "== B2r" >> gpurun_out/ab14.txt; HX_LIB=$PWD/tools/variants/libhx_B2r.so timeout 600 python tools/time_queries.py --sf 1000 --lo-rows 600000000 --reps 3 --queries q3.1,q4.1,q4.3 >> gpurun_out/ab14.txt 2>&1
