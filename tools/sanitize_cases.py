"""Small / ragged invocations of every kernel, for compute-sanitizer runs
(tests/test_sanitizer_gpu.py).  Exits non-zero on a wrong result."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")


def t(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(dev)


def chk(name, got, ref, mag):
    ok, margin = oracle.within_tol(got, ref, mag)
    if not ok:
        print(f"FAIL {name}: margin {margin}")
        sys.exit(1)


for n in (0, 5, 1000, 4099, 70000):
    x, y = synth.numpy_uniform(0, 0, n), synth.numpy_uniform(1, 0, n)
    chk(f"dot{n}", [lift.lift_dot(t(x), t(y)).item()], *[[v] for v in oracle.dot(x, y)])
for m, n in ((7, 3), (5, 129), (33, 4096), (3, 1000), (9, 8192), (2, 20000)):
    A, B = synth.numpy_matrix_rows(2, n, 0, m), synth.numpy_matrix_rows(3, n, 0, m)
    x = synth.numpy_uniform(0, 0, n)
    chk(f"gemv{m}x{n}", lift.lift_gemv(t(A), t(x)).cpu().numpy(), *oracle.gemv(A, x))
    chk(f"gesummv{m}x{n}", lift.lift_gesummv(1.5, t(A), 1.2, t(B), t(x)).cpu().numpy(),
        *oracle.gesummv(1.5, A, 1.2, B, x))
    ref, mag = oracle.atax(A, x)
    for algo in ("auto", "twopass") + (("fused",) if n % 4 == 0 and n <= 16384 else ()):
        chk(f"atax{m}x{n}{algo}", lift.lift_atax(t(A), t(x), algo=algo).cpu().numpy(), ref, mag)
# (600 x 12288, 7 x 8196: 8 float4 columns per thread with x in shared memory, ragged slices)
for m, n in ((40, 32), (200, 4096), (300, 8192), (600, 12288), (7, 8196)):
    A = synth.numpy_matrix_rows(2, n, 0, m)
    x = synth.numpy_uniform(0, 0, n)
    chk(f"atax-fused{m}x{n}", lift.lift_atax(t(A), t(x), algo="fused").cpu().numpy(), *oracle.atax(A, x))
# wide rows: the thread-block-cluster single pass.  600 rows make every cluster refill its ring slots,
# which the last warp done with a slot does after an atom.acq_rel.cta hand-off on a shared counter:
# racecheck does not model that hand-off (it flags every refill against the earlier reads of the slot,
# which all precede the counter's final increment), so under racecheck the refill case is skipped;
# memcheck / synccheck / initcheck run it.
WIDE = ((9, 20000), (40, 32768), (6, 65536)) + (() if os.environ.get("LIFT_SANITIZER_TOOL") == "racecheck"
                                               else ((600, 20000),))
for m, n in WIDE:
    A = synth.numpy_matrix_rows(2, n, 0, m)
    x = synth.numpy_uniform(0, 0, n)
    chk(f"atax-fused-wide{m}x{n}", lift.lift_atax(t(A), t(x), algo="fused").cpu().numpy(), *oracle.atax(A, x))
torch.cuda.synchronize()
print("sanitize cases ok")
