#!/bin/bash
# Round-end evidence on one B200: parity tests (incl. full-size), smoke, a bench line per
# config, ncu launch lists (per-launch DRAM traffic) and full captures of the top kernels.
tag=${1:-final}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${tag}_smi.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${tag}_smoke.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_smoke.log
timeout 400 python bench.py > gpurun_out/${tag}_bench_heat2d5.json 2> gpurun_out/${tag}_bench.err
timeout 300 python bench.py --impl reference > gpurun_out/${tag}_bench_reference.json 2>> gpurun_out/${tag}_bench.err
for c in heat2d9 fdtd2d heat3d gradient3d jacobi2d; do
  timeout 400 python bench.py --config $c > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
if [ -n "$NCU" ]; then
  for c in $NCU; do
    timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
      --csv --log-file gpurun_out/launches_$c.csv python tools/run_once.py $c 1 > gpurun_out/${tag}_ncu_$c.log 2>&1
  done
fi
if [ -n "$NCUFULL" ]; then
  for kc in $NCUFULL; do
    k=${kc%%:*}; c=${kc##*:}
    timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 10 -c 1 \
      -o gpurun_out/${tag}_full_$c python tools/run_once.py $c 1 > gpurun_out/${tag}_ncufull_$c.log 2>&1
  done
fi
