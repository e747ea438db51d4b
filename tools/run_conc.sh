#!/bin/bash
# GPU tests + bench (serial default, then concurrent analytics)
mkdir -p gpurun_out
python -m pytest tests -q -x -m "gpu" 2>&1 | tail -5 > gpurun_out/pt.txt
python bench.py --no-sweep --no-cpu-baseline > gpurun_out/b_serial.json 2> gpurun_out/b_serial.err
python bench.py --no-sweep --no-cpu-baseline --concurrent-analytics > gpurun_out/b_conc.json 2> gpurun_out/b_conc.err
