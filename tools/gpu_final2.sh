#!/bin/bash
# Round-2 final evidence on one B200 (session 2): GPU tests, smoke, ncu launch lists (DRAM / L2 / CTAs per launch -> traffic_*.json) of the
# configs whose kernels changed (first, so the bench lines read their traffic), bench lines for every
# config, the reference arm, and full captures of the top kernels.
tag=${1:-r2f}
mkdir -p gpurun_out/$tag
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/$tag/smi.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/$tag/pytest_gpu.txt 2>&1; echo "pytest rc=$?" >> gpurun_out/$tag/pytest_gpu.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$tag/smoke.txt 2>&1; echo "rc=$?" >> gpurun_out/$tag/smoke.txt
M=dram__bytes_read.sum,dram__bytes_write.sum,lts__t_bytes.sum,gpu__time_duration.sum,launch__grid_size
for c in ${CFGS:-heat2d5 heat2d9 gradient2d fdtd2d heat3d gradient3d heat3d27}; do
  timeout 1200 ncu --metrics $M --clock-control none -k regex:"fast2d|fdtd|fast3d|stream3d|generic|naive" --csv \
    --log-file gpurun_out/$tag/launches_$c.csv python tools/run_once.py $c 1 > gpurun_out/$tag/run_$c.log 2>&1
  python tools/ncu_traffic.py $c gpurun_out/$tag/launches_$c.csv > /dev/null 2> gpurun_out/$tag/tr_$c.err && echo "$c ok" >> gpurun_out/$tag/traffic.log || echo "$c FAIL" >> gpurun_out/$tag/traffic.log
  cp profiles/round2/traffic_$c.json gpurun_out/$tag/ 2>/dev/null
done
timeout 600 python bench.py > gpurun_out/$tag/bench_heat2d5.json 2> gpurun_out/$tag/bench.err
timeout 400 python bench.py --impl reference > gpurun_out/$tag/bench_reference.json 2>> gpurun_out/$tag/bench.err
for c in heat2d9 gradient2d fdtd2d heat3d gradient3d heat3d27 jacobi2d heat3d1024; do
  timeout 600 python bench.py --config $c > gpurun_out/$tag/bench_$c.json 2>> gpurun_out/$tag/bench.err
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fast2d_kernel_v -s 20 -c 1 \
  -o gpurun_out/$tag/full_fast2d_heat2d5 python tools/run_once.py heat2d5 1 > gpurun_out/$tag/ncufull_2d.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fdtd_kernel -s 20 -c 1 \
  -o gpurun_out/$tag/full_fdtd python tools/run_once.py fdtd2d 1 > gpurun_out/$tag/ncufull_fdtd.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:fast3d_kernel -s 10 -c 1 \
  -o gpurun_out/$tag/full_fast3d_heat3d python tools/run_once.py heat3d 1 > gpurun_out/$tag/ncufull_3d.log 2>&1
