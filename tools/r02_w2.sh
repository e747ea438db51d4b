timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py tests/test_gpu_edge_cases.py -m gpu -q -x > gpurun_out/w2_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/w2_tests.txt
for kv in "X=1" "GPMA_ILP=4"; do echo "$kv $(env $kv timeout 300 python tools/upd_probe.py --slides 25 2>&1 | tail -1 | cut -c1-100)" >> gpurun_out/w2_upd.txt; done
bash tools/r02_small_probe.sh w2
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --kernel-name-base function -k regex:"k_lazy_delete_r|k_locate_u_r|k_ins_leaf_u" -c 30 --csv --log-file gpurun_out/w2_upd_launches.csv python tools/upd_probe.py --slides 8 > /dev/null 2>&1
