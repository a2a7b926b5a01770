"""Where the fused ATAX kernel's time goes (tuning aid; the library is not changed).

For each phase P, a patched copy of the package is built under /tmp whose
k_atax_fused stops after that phase:
  1  main loop only (the partial-row store kept behind a runtime-false guard,
     so the rank-1 updates are not dead code)
  2  + store of the per-block partial y row
  3  + grid barrier
  4  + fixed-order column sum (= the library)
  5  phase 2, then the partial row's L2 lines discarded (discard.global.L2): is
     the store's cost the later DRAM write-back of the dirty lines?
  6  the library with the partial-row discards switched off
Phases 4 and 6 also time the two-pass ATAX and the transposed SGEMV.
and lift_atax(algo="fused") is timed (CUDA graph of back-to-back calls, every
call on its own copy of A, copies > 2x L2).
usage: python tools/atax_phase_probe.py
"""
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PKG = "paper_conf_cgo_steuwerrd17_b200"

STORE = "        if (c < nv) P4[c] = yr[q];\n"
AFTER_STORE = "    // ---- second stage in the same launch"
AFTER_BARRIER = "    // every block sums its own slice of columns"

TIMER = r'''
import os, sys
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import torch, synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
for m, n in ((8192, 8192), (148, 8192), (16384, 8192), (4096, 4096)):
    sets = max(2, int(-(-2 * l2 // (4 * m * n))) + 1)
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    calls = [(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 24)[:24]]
    t = graph_time(calls)
    print(f"phase {os.environ['PHASE']} atax {m}x{n}: {t:8.2f} us", flush=True)
    if os.environ["PHASE"] in ("4", "6"):
        t = graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="twopass")) for A in (As * 24)[:24]])
        print(f"        atax twopass {m}x{n}: {t:8.2f} us", flush=True)
        xt = synth.torch_uniform(1, 0, m, device=dev)
        t = graph_time([(lambda A=A: lift.lift_sgemv(1.0, A, xt, 0.0, y=y, trans=True)) for A in (As * 24)[:24]])
        print(f"        sgemv_t {m}x{n}: {t:8.2f} us", flush=True)
    if os.environ["PHASE"] == "4":  # reference: GEMV over the same copies of A
        yg = torch.empty(m, device=dev)
        t = graph_time([(lambda A=A: lift.lift_gemv(A, x, out=yg)) for A in (As * 24)[:24]])
        print(f"        gemv {m}x{n}: {t:8.2f} us", flush=True)
    del As
'''


def patched(phase: int) -> str:
    d = f"/tmp/atax_phase{phase}"
    shutil.rmtree(d, ignore_errors=True)
    os.makedirs(d)
    for sub in (PKG, "include", "synth", "tools"):
        shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                        ignore=shutil.ignore_patterns("_build", "*.so", "__pycache__"))
    f = os.path.join(d, PKG, "csrc", "atax.cu")
    s = open(f).read()
    assert STORE in s and AFTER_STORE in s and AFTER_BARRIER in s
    if phase == 1:
        s = s.replace(STORE, "        if (c < nv && m == -1) P4[c] = yr[q];\n")
    if phase == 5:
        s = s.replace(AFTER_STORE, """    __syncthreads();
    __threadfence();
    for (int64_t l = threadIdx.x; l < nv / 8; l += blockDim.x)  // 128-byte lines of this block's row
        asm volatile("discard.global.L2 [%0], 128;" :: "l"(reinterpret_cast<float4 *>(P) + (int64_t)blockIdx.x * nv + 8 * l) : "memory");
""" + AFTER_STORE)
    if phase == 6:
        old = "return n % 32 == 0 && (reinterpret_cast<uintptr_t>(P) & 127) == 0;"
        assert old in s
        s = s.replace(old, "return false && P && n;")
    if phase in (1, 2, 5):
        s = s.replace(AFTER_STORE, "    if (ex.world == 0) return;  // probe\n" + AFTER_STORE)
    if phase == 3:
        s = s.replace(AFTER_BARRIER, "    if (ex.world == 0) { grid_depart(gbar); return; }  // probe\n" + AFTER_BARRIER)
    open(f, "w").write(s)
    subprocess.run([sys.executable, "-c", f"import sys; sys.path.insert(0, '{d}'); from {PKG} import build; "
                    "build.build(force=True)"], check=True, cwd=d)
    return d


for phase in [int(a) for a in sys.argv[1:]] or (1, 2, 3, 4, 5, 6):
    d = patched(phase)
    subprocess.run([sys.executable, "-c", TIMER], cwd=d, check=True, env=dict(os.environ, PHASE=str(phase)))
