set -x
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "shared_router or host_resident" > gpurun_out/pt_router.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pt_router.log
HX_FORCE_COLLECTIVES=1 timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node=1 --master-addr=127.0.0.1 --master-port=29533 tests/mgpu_worker.py > gpurun_out/mgpu1.log 2>&1; echo "worker rc=$?"; tail -5 gpurun_out/mgpu1.log
