#!/bin/bash
# parity of the touched paths + a warm update launch list + the bench (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_edge_cases.py tests/test_gpu_fullsize.py -m gpu -q -x \
   --deselect tests/test_gpu_fullsize.py::test_config3_halving_full > gpurun_out/${tag}_tests.txt 2>&1
echo "rc=$?" >> gpurun_out/${tag}_tests.txt
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --cache-control none --kernel-name-base function -k regex:"^k_" -c 2000 --csv --log-file gpurun_out/${tag}_warm_launches.csv \
    python tools/upd_probe.py --slides 22 > /dev/null 2>&1
timeout 300 python tools/upd_probe.py --slides 25 > gpurun_out/${tag}_upd.txt 2>&1
timeout 600 python bench.py --no-resize --no-cpu-baseline > gpurun_out/${tag}_bench.json 2> gpurun_out/${tag}_bench.err
