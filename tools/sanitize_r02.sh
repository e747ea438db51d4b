#!/bin/bash
# compute-sanitizer over the round-2 kernels (run under gpurun, 1 GPU): leaf-keyed fused insert,
# interleaved lazy delete, onesweep sort, device-resident level loop, gathers of big windows,
# NCCL dist handle (world size 1), torch allocator hooks, graph replay.
mkdir -p gpurun_out
SEL='config0_sliding_window_lazy[0] or config0_sliding_window_lazy[1] or graph_replay[0] or hot_window or alternative_paths[GPMA_LVL_COOP=0-0] or alternative_paths[GPMA_INS_LEAFSORT=0-0] or random_small_with_resizes[0-1] or random_small_with_resizes[3-0] or sort_tiles_and_stability or torch_allocator or leaf_size_overrides or dist_handle_nccl or example4 or gpma_lock_example2'
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 \
    python -m pytest tests/test_gpu_parity.py tests/test_gpu_edge_cases.py tests/test_gpu_dist.py -q -x \
    -k "$SEL" > gpurun_out/r02_sanitize_$tool.log 2>&1
  echo "$tool exit=$? $(grep -E 'ERROR SUMMARY|passed|failed' gpurun_out/r02_sanitize_$tool.log | tr '\n' ' ')"
done
