#!/bin/bash
# dead-level skip A/B (under gpurun): parity of the level-loop tests, then the configs[3] resize
# trace with the skip off and on
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 900 python -m pytest tests -m gpu -x -q -k "dead_level or config3 or level or resize or parity or edge" > gpurun_out/skab_tests.log 2>&1
echo "tests_rc=$?"; tail -2 gpurun_out/skab_tests.log
for sk in 0 1; do
  GPMA_LVL_SKIP=$sk timeout 900 python tools/resize_trace.py 3 > gpurun_out/skab_rz_$sk.txt 2>&1
  echo "skip=$sk"; grep -v "^    k_" gpurun_out/skab_rz_$sk.txt | tail -6
done
