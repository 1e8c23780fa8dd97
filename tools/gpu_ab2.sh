mkdir -p gpurun_out
bash tools/ab_libs.sh 100 tools/variants/libhx_r01.so paper_journals_pvldb_chrysogeloskaa19_b200/libhx.so tools/variants/libhx_nohint.so tools/variants/libhx_gather0.so tools/variants/libhx_noclaim.so tools/variants/libhx_sleep20.so > gpurun_out/ab2_sf100.txt 2>&1
