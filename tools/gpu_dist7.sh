mkdir -p gpurun_out/r2p
for P in 2 4 8; do
  r=$((P/2))
  HEXS_DIST_EMULATE=3 HEXS_DIST_EMULATE_RANK=$r/$P timeout 300 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2p/emu3_P$P.json 2>gpurun_out/r2p/emu3_P$P.err
  python -c "
import json
d=json.loads(open('gpurun_out/r2p/emu3_P$P.json').read().strip().splitlines()[-1]); e=d['emulated_rank']
print('mode 3 (p2p kernels, self-loop)', $P, e['rank'], round(d['ms_per_step'],2), d['config']['local_extents'])"
done
