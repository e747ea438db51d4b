#!/bin/bash
# GPU tests, then an env experiment (args passed to exp_env.sh)
mkdir -p gpurun_out
python -m pytest tests -q -x -m "gpu" 2>&1 | tail -15 > gpurun_out/pt.txt
bash tools/exp_env.sh "$@" 2>&1 | tee gpurun_out/exp_env.txt
