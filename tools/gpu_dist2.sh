set -x
mkdir -p gpurun_out/r2
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -p no:cacheprovider --timeout 300 -k "dist" > gpurun_out/dist_pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/dist_pytest.txt
tail -3 gpurun_out/dist_pytest.txt
timeout 900 python bench.py --config heat3d1024 --steps 3 --warmup 3 --no-cpu > gpurun_out/r2/bench_heat3d1024.json 2> gpurun_out/r2/bench_heat3d1024.err
cat gpurun_out/r2/bench_heat3d1024.json | cut -c1-600
for P in 2 4 8; do
  for r in 0 $((P/2)); do
    HEXS_DIST_EMULATE_RANK=$r/$P timeout 900 python bench.py --config heat3d1024 --steps 3 --warmup 3 --no-cpu > gpurun_out/r2/emu_heat3d1024_r${r}_P$P.json 2>/dev/null
  done
done
grep -h emulated gpurun_out/r2/emu_*.json | python -c "
import json,sys
for l in sys.stdin:
    d=json.loads(l); e=d['emulated_rank']; print(e['rank'],e['nranks'],round(d['ms_per_step'],1),e['owned_planes'], d['config']['time_block'], round(d['config']['ghost_fraction'],3))"
