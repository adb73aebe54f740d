#!/bin/bash
# 2D profile: tile sweeps of heat2d5 / heat2d9 and one full ncu capture of the star kernel.
tag=${1:-p2d}
mkdir -p gpurun_out
for t in 3,7 3,9 3,10 2,7 2,9 3,5; do
  timeout 200 python bench.py --config heat2d5 --no-cpu --tile $t --steps 5 >> gpurun_out/${tag}_sweep5.json 2>> gpurun_out/${tag}_bench.err
done
for t in 2,7 3,7 2,9 3,5 2,5; do
  timeout 200 python bench.py --config heat2d9 --no-cpu --tile $t --steps 5 >> gpurun_out/${tag}_sweep9.json 2>> gpurun_out/${tag}_bench.err
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:fast2d_kernel_v -s 20 -c 1 \
  -o gpurun_out/${tag}_fast2d python tools/run_once.py heat2d5 1 > gpurun_out/${tag}_ncu.log 2>&1
