#!/bin/bash
# Same-box A/B of one library build under two environment settings (experiment
# switches read by the library), alternating A, B, A, B so drift shows.
# usage: bash tools/ab_env.sh "VAR=a" "VAR=b" script.py [args...]
A=$1; B=$2; shift 2
for rep in 1 2; do
  echo "== $A ($rep)"; env $A python "$@"
  echo "== $B ($rep)"; env $B python "$@"
done
