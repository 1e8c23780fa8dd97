# quick GPU check: plan print, bench (no e2e / cpu baseline), then GPU tests
mkdir -p gpurun_out
HX_DEBUG=1 timeout 300 python tools/prof_query.py --sf 10 --queries all --reps 1 2>&1 | grep K1 > gpurun_out/plans.log
timeout 600 python bench.py --steps 20 --no-e2e --no-cpu-baseline > gpurun_out/bq.json 2> gpurun_out/bq.err; echo "bench rc=$?"
python - <<'PY'
import json
d=json.load(open('gpurun_out/bq.json'))
print('value %.1f G rows/s step %.3f ms frac %.3f moved %.3f' % (d['value']/1e9, d['ms_per_step'], d['roofline']['frac'], d['roofline']['frac_moved']))
print(' '.join(f"{q[1:]}:{v['k1_ms']*1e3:.0f}" for q, v in d['per_query'].items()))
PY
if [ "$1" = "test" ]; then timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -3; fi
