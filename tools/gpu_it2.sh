#!/bin/bash
tag=${1:-it2}
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "fdtd or 2d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in fdtd2d heat2d5 heat2d9; do
  timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
for t in 2,8 2,6 2,7; do
  timeout 200 python bench.py --config heat2d5 --no-cpu --tile $t --steps 5 >> gpurun_out/${tag}_sweep5.json 2>> gpurun_out/${tag}_bench.err
done
