#!/bin/bash
# row-search interpolation A/B (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_edge_cases.py tests/test_gpu_fullsize.py -m gpu -q -x \
   --deselect tests/test_gpu_fullsize.py::test_config3_halving_full > gpurun_out/${tag}_tests.txt 2>&1
echo "rc=$?" >> gpurun_out/${tag}_tests.txt
for kv in "GPMA_INTERP=1" "GPMA_INTERP=0" "GPMA_INTERP=1" "GPMA_INTERP=0"; do
  echo "$kv $(env $kv timeout 300 python tools/upd_probe.py --slides 25 2>&1 | tail -1 | cut -c1-100)" >> gpurun_out/${tag}_ab.txt
done
for kv in "GPMA_INTERP=1" "GPMA_INTERP=0"; do
  env $kv timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --kernel-name-base function -k regex:"k_lazy_delete_r|k_locate_u_r" -c 12 --csv --log-file gpurun_out/${tag}_${kv}_ncu.csv \
    python tools/upd_probe.py --slides 6 > /dev/null 2>&1
done
