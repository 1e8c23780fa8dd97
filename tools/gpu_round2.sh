# Round-2 measurement pass: GPU tests, default bench (SF100), launch list, ncu --set full of
# the 13 K1 launches at SF100, probe-table L2 hit rates (evict_last-tagged probe build).
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_gpu.log
timeout 900 python bench.py --steps 20 --warmup 5 > gpurun_out/bench.json 2> gpurun_out/bench.err; echo "bench rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-ht-path > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:"k1_(probe|scan)_agg" -s 13 -c 13 -o gpurun_out/k1_full python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/ncu_full.log 2>&1; echo "ncu2 rc=$?"
HX_LIB=$PWD/tools/variants/libhx_PH.so timeout 900 ncu --clock-control none -k regex:"k1_probe_agg" -s 13 -c 13 --csv --metrics gpu__time_duration.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_miss.sum,lts__t_sectors_srcunit_tex_evict_first_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_first_lookup_miss.sum,lts__t_sectors_srcunit_tex_evict_normal_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_normal_lookup_miss.sum,dram__bytes_read.sum,dram__bytes_write.sum --log-file gpurun_out/probe_l2.csv python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/probe_l2.log 2>&1; echo "ncu3 rc=$?"
HX_LIB=$PWD/tools/variants/libhx_PH.so timeout 900 ncu --clock-control none -k regex:"k1_probe_agg" -s 13 -c 13 --csv --metrics gpu__time_duration.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_miss.sum,dram__bytes_read.sum --log-file gpurun_out/probe_l2_sf1000.csv python tools/prof_query.py --sf 1000 --lo-rows 600000000 --queries all --reps 2 > gpurun_out/probe_l2_sf1000.log 2>&1; echo "ncu4 rc=$?"
