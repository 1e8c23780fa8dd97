mkdir -p gpurun_out
JOIN=hash bash tools/gpu_ncu_q.sh 100 q4.2 gpurun_out/k1_ht_q42
ls -la gpurun_out/k1_ht_q42*
