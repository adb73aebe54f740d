#!/bin/bash
# 3D early In rows: the whole 3D GPU suite (parity incl. full size, tile shapes, dist loopback) + bench.
tag=${1:-ei}
mkdir -p gpurun_out
timeout 120 python -m pytest tests/test_gpu_parity.py -x -q -k "test_3d and star3d7 and float32" > gpurun_out/${tag}_quick.log 2>&1
rc=$?; echo "rc=$rc" >> gpurun_out/${tag}_quick.log
if [ $rc -ne 0 ]; then exit 0; fi
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "3d or dist" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in heat3d heat3d27 gradient3d heat3d1024; do
  timeout 400 python bench.py --config $c --no-cpu > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
