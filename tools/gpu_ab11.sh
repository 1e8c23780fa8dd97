mkdir -p gpurun_out
for lib in tools/variants/libhx_B2r.so tools/variants/libhx_W26.so; do
echo "== $lib"
HX_LIB=$PWD/$lib HX_DEBUG=1 timeout 300 python tools/time_queries.py --sf 10 --reps 5 --queries q4.1,q4.2,q4.3 2>&1
done > gpurun_out/ab11.txt
