#!/bin/bash
# 3D kernel iteration: parity tests for the 3D classes, a heat3d bench line, a tile sweep.
tag=${1:-3d}
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "3d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
timeout 200 python bench.py --config heat3d --no-cpu > gpurun_out/${tag}_bench_heat3d.json 2> gpurun_out/${tag}_bench.err
timeout 200 python bench.py --config gradient3d --no-cpu > gpurun_out/${tag}_bench_gradient3d.json 2>> gpurun_out/${tag}_bench.err
for t in ${TILES:-1,3 2,3 2,5 3,5 3,7 1,7}; do
  timeout 200 python bench.py --config heat3d --no-cpu --tile $t --steps 3 >> gpurun_out/${tag}_sweep.json 2>> gpurun_out/${tag}_bench.err
done
if [ -n "$NCU" ]; then
  timeout 400 ncu --set full --clock-control none --import-source on -k regex:fast3d_kernel -s 10 -c 1 -o gpurun_out/${tag}_fast3d python tools/run_once.py heat3d 1 > gpurun_out/${tag}_ncu.log 2>&1
fi
