#!/bin/bash
# Final verification of the committed build: all GPU tests, smoke, the default bench line and heat-3D.
tag=${1:-vf}
mkdir -p gpurun_out/$tag
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/$tag/pytest_gpu.txt 2>&1; echo "pytest rc=$?" >> gpurun_out/$tag/pytest_gpu.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$tag/smoke.txt 2>&1; echo "rc=$?" >> gpurun_out/$tag/smoke.txt
timeout 600 python bench.py > gpurun_out/$tag/bench_heat2d5.json 2> gpurun_out/$tag/bench.err
timeout 600 python bench.py --config heat3d > gpurun_out/$tag/bench_heat3d.json 2>> gpurun_out/$tag/bench.err
timeout 600 python bench.py --config fdtd2d > gpurun_out/$tag/bench_fdtd2d.json 2>> gpurun_out/$tag/bench.err
