"""Every plausible slip in the oracle is caught by a pin (tools/mutate_oracle.py).

Builds mutated copies of oracle/oracle.c (strided instead of adjacent Listing-1
pairing, inflated `mag`, swapped alpha/beta, transposed ATAX pass 2, dropped
terms, ...) and runs tests/test_oracle_pins.py against each; every mutation
must make at least one pin fail.  CPU only.
"""
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_every_oracle_mutation_is_killed():
    r = subprocess.run([sys.executable, os.path.join(ROOT, "tools", "mutate_oracle.py")],
                       cwd=ROOT, capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "SURVIVED" not in r.stdout
