#!/bin/bash
# Kernel iteration: parity tests for the touched classes and bench lines for their configs.
# usage: tools/gpu_iter.sh TAG "pytest -k expr" "config list"
tag=${1:-it}; kx=${2:-2d}; cfgs=${3:-heat2d5}
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "$kx" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in $cfgs; do
  timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
