#!/bin/bash
# A/B of the fused-ATAX partial-row L2 discard inside bench.py's table1 block
# (tuning aid): the library as built vs a copy built with the discard off
# (tools/atax_phase_probe.py's phase-6 patch).  usage: bash tools/ab_discard.sh OUTDIR
OUT=${1:-gpurun_out/ab}; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
python - <<'PY'
g = {'__file__': 'tools/atax_phase_probe.py'}
src = open('tools/atax_phase_probe.py').read().split('for phase in [int')[0]
exec(src, g)
d = g['patched'](6)
import shutil, os
for f in ('bench.py', 'BASELINE.json', '__graft_entry__.py'):
    shutil.copy(f, d)
shutil.copytree('oracle', os.path.join(d, 'oracle'), dirs_exist_ok=True)
shutil.copytree('profiles', os.path.join(d, 'profiles'), dirs_exist_ok=True)
PY
for rep in 1 2; do
  timeout 600 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu > $OUT/on_$rep.json 2> $OUT/on_$rep.err
  (cd /tmp/atax_phase6 && timeout 600 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu) > $OUT/off_$rep.json 2> $OUT/off_$rep.err
done
python - "$OUT" <<'PY'
import json, sys, glob, os
for f in sorted(glob.glob(os.path.join(sys.argv[1], '*.json'))):
    try:
        d = json.load(open(f))
    except Exception as e:
        print(f, 'ERR', e); continue
    t = d['table1']
    print(os.path.basename(f), d['clocks']['sm_mhz'], 'ops atax', d['ops']['atax_8192x8192']['ms'],
          'table1', {k: t[k]['us'] for k in ('atax_4096x4096', 'atax_8192x8192', 'gemv_4096x4096', 'dot_2^20')})
PY
