#!/bin/bash
# Round-2 re-entry check (under gpurun): build, smoke, every GPU test, the default bench line.
tag=${1:-c0}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/${tag}_build.log 2>&1; echo "build_rc=$?"
timeout 300 python __graft_entry__.py smoke > gpurun_out/${tag}_smoke.log 2>&1; echo "smoke_rc=$?"
timeout 1500 python -m pytest tests -m gpu -x -q --durations=15 > gpurun_out/${tag}_tests.log 2>&1
echo "tests_rc=$?"; tail -20 gpurun_out/${tag}_tests.log
timeout 900 python bench.py --log-jsonl gpurun_out/${tag}_slides.jsonl > gpurun_out/${tag}_bench.json 2> gpurun_out/${tag}_bench.err
echo "bench_rc=$?"; tail -3 gpurun_out/${tag}_bench.err
