# run the SF10 bench under several environment settings: bash tools/gpu_env_sweep.sh "A=1 B=2" "A=3" ...
mkdir -p gpurun_out
for c in "$@"; do
  env $c timeout 300 python bench.py --steps 20 --no-e2e --no-cpu-baseline > gpurun_out/sw.json 2>/dev/null
  python - "$c" <<'PY'
import json, sys
d=json.load(open('gpurun_out/sw.json'))
print(sys.argv[1], 'value %.1f step %.3f frac %.3f' % (d['value']/1e9, d['ms_per_step'], d['roofline']['frac']),
      ' '.join(f"{q[1:]}:{v['k1_ms']*1e3:.0f}" for q, v in d['per_query'].items()))
PY
done
