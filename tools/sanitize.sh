#!/bin/bash
# compute-sanitizer over representative GPU parity tests (run under gpurun, 1 GPU)
mkdir -p gpurun_out
SEL='config0_sliding_window_lazy[0] or config0_sliding_window_rebalance[0] or random_small_with_resizes[0-1] or random_small_with_resizes[1-0] or gpma_lock_example2 or example4'
SEL2='graph_replayed_sliding_window[0-0] or graph_replayed_sliding_window[0-1] or replay_errors or across_resizes[0-0] or every_strategy[10] or every_sample_strategy[10] or level_step_paths'
for tool in memcheck racecheck synccheck; do
  compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 \
    python -m pytest tests/test_gpu_parity.py tests/test_gpu_query.py tests/test_gpu_edge_cases.py \
    tests/test_gpu_update_graph.py tests/test_gpu_bfs_strategies.py -q -x \
    -k "$SEL or $SEL2 or reachability_closed_form or all_duplicates" > gpurun_out/sanitize_$tool.log 2>&1
  echo "$tool exit=$? $(grep -E 'ERROR SUMMARY|passed|failed' gpurun_out/sanitize_$tool.log | tr '\n' ' ')"
done
