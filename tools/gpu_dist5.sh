# halo copy cost (pack / device-local wire / unpack) per rank, y slabs, default tile
mkdir -p gpurun_out/r2x
for P in 2 4 8; do
  r=$((P/2))
  for mode in 1 2; do
    HEXS_DIST_EMULATE=$mode HEXS_DIST_EMULATE_RANK=$r/$P timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2x/emu${mode}_P$P.json 2>gpurun_out/r2x/emu${mode}_P$P.err
    python -c "
import json
d=json.loads(open('gpurun_out/r2x/emu${mode}_P$P.json').read().strip().splitlines()[-1]); e=d['emulated_rank']
print('mode $mode', $P, e['rank'], round(d['ms_per_step'],2), d['config']['local_extents'], d['config']['tile'] if 'tile' in d['config'] else '')"
  done
done
