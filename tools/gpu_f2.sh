#!/bin/bash
# Packed-FP32 (FADD2) iteration: throughput probe, 2D parity tests, 2D bench lines.
tag=${1:-f2}
mkdir -p gpurun_out
./tools/probe_f32x2/probe > gpurun_out/${tag}_probe.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "2d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in heat2d5 heat2d9 jacobi2d; do
  timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
for t in ${TILES:-3,7 3,9 3,10 2,7 2,9}; do
  timeout 200 python bench.py --config heat2d5 --no-cpu --tile $t --steps 5 >> gpurun_out/${tag}_sweep.json 2>> gpurun_out/${tag}_bench.err
done
