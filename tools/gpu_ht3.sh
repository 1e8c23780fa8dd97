mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_hx_gpu.py -x -q -k "instances_and_probe or small_sf or plans_key or probe_order" > gpurun_out/pt_ht3.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pt_ht3.log
JOIN=hash bash tools/ab_env.sh 100 "HX_NONE=1" "HX_HT_FIRST_MIN=99" > gpurun_out/ab35.txt 2>&1
JOIN=hash bash tools/ab_env.sh 10 "HX_NONE=1" "HX_HT_FIRST_MIN=99" "HX_HT_FIRST_MIN=0.2" "HX_HT_FIRST_MIN=0.4" >> gpurun_out/ab35.txt 2>&1
bash tools/ab_libs.sh 100 tools/variants/libhx_SC.so paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so >> gpurun_out/ab35.txt 2>&1
