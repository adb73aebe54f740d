# round-2 full GPU pass: every -m gpu test, then one bench line per config, the reference arm,
# and emulated-rank projections of the slab-partitioned 1024^3 run
set -x
mkdir -p gpurun_out/r2
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider --timeout 900 --durations=20 > gpurun_out/r2/pytest_gpu.txt 2>&1; echo "pytest rc=$?" >> gpurun_out/r2/pytest_gpu.txt
tail -30 gpurun_out/r2/pytest_gpu.txt
for c in heat2d5 heat2d9 gradient2d jacobi2d fdtd2d heat3d gradient3d heat3d27 heat3d1024; do
  timeout 900 python bench.py --config $c --steps 5 --warmup 3 > gpurun_out/r2/bench_$c.json 2> gpurun_out/r2/bench_$c.err
  echo "== $c"; cat gpurun_out/r2/bench_$c.json | cut -c1-400
done
timeout 600 python bench.py --impl reference --steps 5 --warmup 3 > gpurun_out/r2/bench_reference.json 2>&1
for P in 2 4 8; do
  for r in 0 $((P/2)); do
    HEXS_DIST_EMULATE_RANK=$r/$P timeout 900 python bench.py --config heat3d1024 --steps 3 --warmup 3 --no-cpu > gpurun_out/r2/emu_heat3d1024_r${r}_P$P.json 2>/dev/null
  done
done
grep -h emulated gpurun_out/r2/emu_*.json | python -c "
import json,sys
for l in sys.stdin:
    d=json.loads(l); e=d['emulated_rank']; print(e['rank'],e['nranks'],d['ms_per_step'],e['owned_planes'])"
