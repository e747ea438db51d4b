#!/bin/bash
# device level loop on / off and CTAs per SM: the configs[3] resize stress (grow phase has 0.6M
# updates past the leaves near each doubling)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for kv in "X=1" "GPMA_LVL_COOP=0" "GPMA_COOP_CTAS=1" "GPMA_COOP_CTAS=4"; do
  env $kv timeout 900 python bench.py --steps 3 --warmup 3 --no-sweep --no-cpu-baseline --no-e2e > gpurun_out/co_$kv.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/co_$kv.json').read().strip().splitlines()[-1]); r=d['resize_stress']
print('$kv', 'step %.3f' % d['ms_per_step'], 'resize', r['ms_resize_steps'], 'mean %.3f' % r['ms_per_step_mean'], 'other %.3f' % r['ms_other_step_mean'])"
done
