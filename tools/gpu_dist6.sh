mkdir -p gpurun_out/r2x
timeout 600 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "dist" -p no:cacheprovider > gpurun_out/r2x/pytest_dist.txt 2>&1; tail -2 gpurun_out/r2x/pytest_dist.txt
for P in 2 4 8; do
  r=$((P/2))
  HEXS_DIST_EMULATE=2 HEXS_DIST_EMULATE_RANK=$r/$P timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2x/emu2b_P$P.json 2>gpurun_out/r2x/emu2b_P$P.err
  python -c "
import json
d=json.loads(open('gpurun_out/r2x/emu2b_P$P.json').read().strip().splitlines()[-1]); e=d['emulated_rank']
print('mode 2 rows', $P, e['rank'], round(d['ms_per_step'],2), d['config']['local_extents'])"
done
timeout 900 python bench.py --config heat3d1024 --steps 3 --warmup 3 > gpurun_out/r2x/n1.json 2>gpurun_out/r2x/n1.err; cut -c1-300 gpurun_out/r2x/n1.json
