#!/bin/bash
# Level-loop warp-merge A/B (under gpurun): tests of the touched paths, 25 configs[2] slides and
# configs[3] ordinary steps with GPMA_LVL_WARP on / off.   tools/r02_warp_ab.sh <tag>
tag=${1:-x}
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_bfs_strategies.py tests/test_gpu_dist.py \
    tests/test_gpu_edge_cases.py -m gpu -q -x > gpurun_out/${tag}_tests.txt 2>&1
echo "tests_rc=$?" >> gpurun_out/${tag}_tests.txt
for kv in "GPMA_LVL_WARP=1" "GPMA_LVL_WARP=0" "GPMA_LVL_COOP=0"; do
  echo "$kv $(env $kv timeout 300 python tools/upd_probe.py --slides 25 2>&1 | tail -1 | cut -c1-160)" >> gpurun_out/${tag}_warp.txt
done
for kv in "GPMA_LVL_WARP=1" "GPMA_LVL_WARP=0" "GPMA_LVL_COOP=0 GPMA_LVL_SMALL=0"; do
  echo "$kv $(env $kv timeout 300 python tools/resize_steps_ab.py --grow 40 2>&1 | tail -1)" >> gpurun_out/${tag}_c3.txt
done
timeout 300 python bench.py --no-sweep --no-resize --no-cpu-baseline > gpurun_out/${tag}_bench.txt 2>&1
