#!/bin/bash
# A/B helper (under gpurun): build, selected GPU tests, then the bench (no sweep / resize / e2e)
# once per "ENV=VAL" argument ("-" = defaults).
# usage: tools/r02c_ab.sh <tag> "<pytest -k expr or ->" [env settings ...]
tag=$1; kexpr=$2; shift 2
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/${tag}_build.log 2>&1 || { echo build failed; tail -20 gpurun_out/${tag}_build.log; exit 1; }
if [ "$kexpr" != "-" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q -k "$kexpr" > gpurun_out/${tag}_tests.log 2>&1
  echo "tests_rc=$?"; tail -3 gpurun_out/${tag}_tests.log
fi
for kv in "$@"; do
  n=$(echo "$kv" | tr '=' '_' | tr -d ' ')
  if [ "$kv" = "-" ]; then e=""; else e="$kv"; fi
  env $e timeout 600 python bench.py --steps 20 --warmup 5 --no-sweep --no-resize --no-cpu-baseline --no-e2e > gpurun_out/${tag}_${n}.json 2> gpurun_out/${tag}_${n}.err
  echo "bench[$kv] rc=$?"
  python - "$kv" gpurun_out/${tag}_${n}.json <<'PY'
import json, sys
try:
    d = json.loads(open(sys.argv[2]).read().strip().splitlines()[-1])
    print(sys.argv[1], "ms/step %.3f" % d["ms_per_step"], {k: round(v, 4) for k, v in d["breakdown_ms"].items() if isinstance(v, float)},
          "upd %.4f" % d["update_only"]["ms_per_slide"])
except Exception as ex:
    print(sys.argv[1], "no result", ex)
PY
done
