#!/bin/bash
# Round-2 evidence, final pass (under gpurun, 1 GPU): GPU tests, the default bench line, a
# per-slide log, the warm launch list of one bench step, ncu --set full of the heavy kernels.
tag=${1:-r02c}
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -q -x > gpurun_out/${tag}_gputests.log 2>&1
echo "tests_rc=$?" >> gpurun_out/${tag}_gputests.log
timeout 1500 python bench.py --log-jsonl gpurun_out/${tag}_slides.jsonl > gpurun_out/${tag}_bench.json 2> gpurun_out/${tag}_bench.err
echo "bench_rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --cache-control none --kernel-name-base function -k regex:"^k_" -c 3000 --csv --log-file gpurun_out/${tag}_launches.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/${tag}_launches_bench.log 2>&1
echo "launches_rc=$?"
timeout 1200 ncu --set full --clock-control none --import-source on \
    -k regex:"k_pr_push_win|k_exp_tma|k_cc_hook|k_bfs_sweep|k_ins_leaf_u|k_lazy_delete_r|k_os_pass|k_locate_u_r|k_pr_step|k_cc_sample|k_levels_coop|k_group_starts|k_layout_even|k_lvl_gather_big" \
    -s 60 -c 16 -o gpurun_out/${tag}_full python bench.py --steps 1 --warmup 2 --no-e2e --no-cpu-baseline --no-sweep --no-resize \
    > gpurun_out/${tag}_full.log 2>&1
echo "full_rc=$?"
