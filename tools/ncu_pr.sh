#!/bin/bash
# ncu --set full of the PageRank push variants (one GPU)
mkdir -p gpurun_out
for cfg in "$@"; do
GPMA_PR_CFG=$cfg ncu --set full --clock-control none --import-source on --kernel-name-base function \
    -k regex:"k_pr_push" -s 2 -c 1 -o gpurun_out/pr_cfg$cfg \
    python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep > gpurun_out/ncu_pr_$cfg.log 2>&1
done
GPMA_PR_TMA=0 ncu --set full --clock-control none --import-source on --kernel-name-base function \
    -k regex:"k_pr_push" -s 2 -c 1 -o gpurun_out/pr_win \
    python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep > gpurun_out/ncu_pr_win.log 2>&1
