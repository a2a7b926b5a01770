#!/bin/bash
# A/B of the fused ATAX kernel: this tree vs the tree exported under ab_old/
# (git archive <rev> | tar -x -C ab_old; untracked, travels with gpurun).
# Prints both timings and whether the outputs are bitwise equal.
# usage: bash tools/ab_atax.sh OUTDIR
OUT=${1:-gpurun_out/ab_atax}; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build_new.log 2>&1 || exit 1
(cd ab_old && python -c "import __graft_entry__ as g; g.build()") > $OUT/build_old.log 2>&1 || exit 1
for rep in 1 2; do
  echo "== new ($rep)"; python tools/ab_atax.py $OUT/new.npz
  echo "== old ($rep)"; (cd ab_old && python ../tools/ab_atax.py ../$OUT/old.npz)
done
python - $OUT <<'PY'
import sys, numpy as np
a, b = np.load(sys.argv[1] + '/new.npz'), np.load(sys.argv[1] + '/old.npz')
for k in a.files:
    if k.startswith('y_'):
        print(k, 'bitwise equal' if np.array_equal(a[k].view(np.uint32), b[k].view(np.uint32)) else 'DIFFERENT')
PY
