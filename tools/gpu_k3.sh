mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hashjoin_gpu.py -x -q > gpurun_out/pt_k3.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pt_k3.log
for e in "HX_K3_LDG=1" "HX_X=1"; do echo "== $e"; env $e timeout 600 python tools/hashpack_bench.py --sf 100 --parts 8 2>&1 | tail -1; done > gpurun_out/k3ab.txt
for p in 2 64; do echo "== parts $p"; timeout 600 python tools/hashpack_bench.py --sf 100 --parts $p 2>&1 | tail -1; done >> gpurun_out/k3ab.txt
