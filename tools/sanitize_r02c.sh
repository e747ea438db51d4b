#!/bin/bash
# compute-sanitizer, final round-2 pass (run under gpurun, 1 GPU): the kernels added in the last
# session -- dead-level skip (k_lvl_first_accept), one-pass group starts (k_group_starts), the root
# re-layout writing the heads, the block cache (allocation reuse across resizes) -- plus the
# configs[0] sweep on both batch paths and the scaled configs[3] resize stress.
mkdir -p gpurun_out
tag=${1:-r02c}
T=tests/test_gpu_parity.py
E=tests/test_gpu_edge_cases.py
F=tests/test_gpu_fullsize.py
SEL="$E::test_dead_level_skip_intermediate_and_root[0] $E::test_dead_level_skip_intermediate_and_root[1] $T::test_config0_sliding_window_lazy[0-small] $T::test_config0_sliding_window_lazy[0-large] $T::test_config0_alternative_paths[0-GPMA_GSTART_FUSED=0] $T::test_config0_alternative_paths[0-GPMA_LVL_SKIP=0] $T::test_random_small_with_resizes[0-1] $E::test_sort_tiles_and_stability[4097] $E::test_oversized_leaf_groups[1] $F::test_config3_resize_stress_scaled"
for tool in memcheck racecheck synccheck; do
  timeout 2400 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 \
    python -m pytest $SEL -q -x > gpurun_out/${tag}_sanitize_$tool.log 2>&1
  echo "$tool exit=$? $(grep -E 'ERROR SUMMARY|passed|failed' gpurun_out/${tag}_sanitize_$tool.log | tr '\n' ' ')"
done
