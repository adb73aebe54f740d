# y-partitioned slab mode: NCCL single-rank test, N=1 dist bench, emulated ranks per tile
mkdir -p gpurun_out/r2y
timeout 600 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "dist" -p no:cacheprovider > gpurun_out/r2y/pytest_dist.txt 2>&1; tail -2 gpurun_out/r2y/pytest_dist.txt
timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2y/n1.json 2> gpurun_out/r2y/n1.err
python -c "
import json; d=json.loads(open('gpurun_out/r2y/n1.json').read().strip().splitlines()[-1]); print('N=1', d['config']['partition'], d['config'].get('local_extents'), round(d['ms_per_step'],1), round(d['value'],1), d['e2e']['value'])"
for t in 2,7 3,7 2,5; do
  for P in 2 4 8; do
    r=$((P/2))
    HEXS_DIST_EMULATE_RANK=$r/$P timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu --tile $t > gpurun_out/r2y/emu_${t}_P$P.json 2>gpurun_out/r2y/emu_${t}_P$P.err
    python -c "
import json
d=json.loads(open('gpurun_out/r2y/emu_${t}_P$P.json').read().strip().splitlines()[-1]); e=d['emulated_rank']
print('$t', $P, e['rank'], round(d['ms_per_step'],1), e['owned_indices'], d['config']['local_extents'], round(d['config']['ghost_fraction'],3))"
  done
done
HEXS_DIST_EMULATE_RANK=0/8 timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2y/emu_def_r0_P8.json 2>/dev/null
python -c "
import json
d=json.loads(open('gpurun_out/r2y/emu_def_r0_P8.json').read().strip().splitlines()[-1]); print('edge r0 P8', round(d['ms_per_step'],1), d['config']['local_extents'])"
