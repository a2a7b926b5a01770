#!/bin/bash
# Same-box A/B of this tree against an older tree exported under ab_old/
# (git archive <rev> | tar -x -C ab_old; untracked, travels with gpurun): builds
# both, then runs THIS tree's script with LIFT_ROOT pointing at each package
# root, alternating new, old, new, old so drift shows.
# usage: bash tools/ab_tree.sh tools/atax_time.py [args...]
python -c "import __graft_entry__ as g; g.build()" > /tmp/ab_build_new.log 2>&1 || { tail -20 /tmp/ab_build_new.log; exit 1; }
(cd ab_old && python -c "import __graft_entry__ as g; g.build()") > /tmp/ab_build_old.log 2>&1 || { tail -20 /tmp/ab_build_old.log; exit 1; }
for rep in 1 2; do
  echo "== new ($rep)"; LIFT_ROOT=$(pwd) python "$@"
  echo "== old ($rep)"; LIFT_ROOT=$(realpath ab_old) python "$@"
done
