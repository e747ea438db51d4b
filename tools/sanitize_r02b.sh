#!/bin/bash
# compute-sanitizer, second round-2 pass (run under gpurun, 1 GPU): both batch paths of the
# configs[0] sweep, the one-kernel small insert (merge sort, cooperative leaf I/O) and the
# multi-CTA small delete, the warp / CTA merges of the cooperative level loop, the pending
# segment sort, the interpolated row search, in-place large batches, NCCL world size 1.
mkdir -p gpurun_out
tag=${1:-r02b}
T=tests/test_gpu_parity.py
E=tests/test_gpu_edge_cases.py
SEL="$T::test_config0_sliding_window_lazy[0-small] $T::test_config0_sliding_window_lazy[0-large] $T::test_config0_sliding_window_graph_replay[0] $T::test_sorted_stream_hot_window[0-1] $T::test_sorted_stream_hot_window[1-1-blockmerge] $T::test_config0_alternative_paths[0-GPMA_LVL_WARP=0] $T::test_config0_alternative_paths[0-GPMA_INTERP=0] $T::test_config0_alternative_paths[0-GPMA_SMALL=2048] $T::test_random_small_with_resizes[0-1] $T::test_example4_on_gpu $T::test_gpma_lock_example2_on_gpu $T::test_pagerank_push_strategies[0] $E::test_small_path_sizes_and_stability[2048] $E::test_small_path_sizes_and_stability[65] $E::test_multi_cta_small_delete_rejects_whole_batch[1500] $E::test_large_device_batch_direct_vs_staged[1] $E::test_sort_tiles_and_stability[4097] $E::test_oversized_leaf_groups[1] tests/test_gpu_dist.py::test_dist_handle_nccl_world_one[0]"
for tool in memcheck racecheck synccheck; do
  timeout 1800 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 \
    python -m pytest $SEL -q -x > gpurun_out/${tag}_sanitize_$tool.log 2>&1
  echo "$tool exit=$? $(grep -E 'ERROR SUMMARY|passed|failed' gpurun_out/${tag}_sanitize_$tool.log | tr '\n' ' ')"
done
