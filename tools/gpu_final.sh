# Round-2 final measurement pass (the .ncu-rep files are summarised on the box and removed:
# gpurun copies back at most 64 MiB).
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
( time timeout 900 python bench.py --steps 20 --warmup 5 > gpurun_out/bench.json 2> gpurun_out/bench.err ) 2> gpurun_out/bench_time.txt; echo "bench rc=$?"
timeout 600 python bench.py --impl reference --steps 20 --warmup 5 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err; echo "ref rc=$?"
timeout 600 python bench.py --sf 10 --steps 20 --warmup 5 --no-e2e > gpurun_out/bench_sf10.json 2> gpurun_out/bench_sf10.err; echo "sf10 rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-ht-path > gpurun_out/b_ncu.log 2>&1; echo "ncu1 rc=$?"
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:"k1_(probe|scan)_agg" -s 13 -c 13 -o /tmp/k1_full python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/ncu_full.log 2>&1; echo "ncu2 rc=$?"
ncu -i /tmp/k1_full.ncu-rep --page raw --csv > gpurun_out/k1_full_raw.csv 2>/dev/null
for i in 3 6 10; do python tools/ncu_lines.py /tmp/k1_full.ncu-rep --launch $i --rows 6e8 --top 40 > gpurun_out/k1_lines_$i.txt 2>&1; done
HX_LIB=$PWD/tools/variants/libhx_PH.so timeout 900 ncu --clock-control none -k regex:"k1_probe_agg" -s 13 -c 13 --csv --metrics gpu__time_duration.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_last_lookup_miss.sum,lts__t_sectors_srcunit_tex_evict_first_lookup_hit.sum,lts__t_sectors_srcunit_tex_evict_first_lookup_miss.sum,dram__bytes_read.sum --log-file gpurun_out/probe_l2.csv python tools/prof_query.py --sf 100 --queries all --reps 2 > gpurun_out/probe_l2.log 2>&1; echo "ncu3 rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k3_" -c 3 -o /tmp/k3_full python tools/hashpack_bench.py --sf 100 --parts 8 --reps 1 > gpurun_out/k3_ncu.log 2>&1; echo "ncu4 rc=$?"
ncu -i /tmp/k3_full.ncu-rep --page raw --csv > gpurun_out/k3_full_raw.csv 2>/dev/null
timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 > gpurun_out/hashpack.jsonl 2> gpurun_out/hashpack.err; echo "hashpack rc=$?"
du -sh gpurun_out
