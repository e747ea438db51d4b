#!/bin/bash
# compute-sanitizer over the round-2 kernels (run under gpurun, 1 GPU): leaf-keyed fused insert,
# interleaved lazy delete, onesweep sort, device-resident level loop, gathers of big windows,
# NCCL dist handle (world size 1), torch allocator hooks, graph replay.
mkdir -p gpurun_out
T=tests/test_gpu_parity.py
E=tests/test_gpu_edge_cases.py
SEL="$T::test_config0_sliding_window_lazy[0] $T::test_config0_sliding_window_lazy[1] $T::test_config0_sliding_window_graph_replay[0] $T::test_sorted_stream_hot_window $T::test_config0_alternative_paths[0-GPMA_LVL_COOP=0] $T::test_config0_alternative_paths[0-GPMA_SMALL=2048] $T::test_config0_alternative_paths[0-GPMA_INS_LEAFSORT=0] $T::test_random_small_with_resizes[0-1] $T::test_random_small_with_resizes[3-0] $T::test_example4_on_gpu $T::test_gpma_lock_example2_on_gpu $T::test_pagerank_push_strategies[0] $E::test_sort_tiles_and_stability[4097] $E::test_torch_allocator_hooks $E::test_leaf_size_overrides tests/test_gpu_dist.py::test_dist_handle_nccl_world_one[0]"
for tool in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 \
    python -m pytest $SEL -q -x > gpurun_out/r02_sanitize_$tool.log 2>&1
  echo "$tool exit=$? $(grep -E 'ERROR SUMMARY|passed|failed' gpurun_out/r02_sanitize_$tool.log | tr '\n' ' ')"
done
