#!/bin/bash
# bench each tuning build of libhx (K1 warps/CTA x CTAs/SM); prints per-query K1 GB/s
for lib in paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so tools/variants/libhx_*.so; do
  HX_LIB=$PWD/$lib timeout 300 python bench.py --steps 5 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/var.json 2>gpurun_out/var.err
  python - "$lib" <<'PY'
import json, sys
d = json.load(open('gpurun_out/var.json'))
pq = d['per_query']
print(sys.argv[1].split('/')[-1], f"{d['value']/1e9:.1f} Grows/s step {d['ms_per_step']:.2f} ms K1 frac {d['roofline']['frac']:.3f} ctas {d['k1_ctas_per_sm']}",
      ' '.join(f"{q[1:]}:{v['k1_frac_of_peak']:.2f}" for q, v in pq.items()))
PY
done
