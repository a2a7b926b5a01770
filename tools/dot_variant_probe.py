"""k_dot launch / second-stage variants at small n (tuning aid; the library is not changed).

Each variant is a copy of the package under /tmp with textual patches to
csrc/dot.cu, built and timed at n = 2^20, 2^22, 2^24 (graph of >= 20 calls
over distinct slices totalling > 2x L2, best of 3 replays).  "nofinal" drops
the ticket and the second stage (wrong result; shows what they cost).
usage: python tools/dot_variant_probe.py [name ...]
"""
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SRC = os.path.join(ROOT, "paper_conf_cgo_steuwerrd17_b200", "csrc", "dot.cu")

VARIANTS = {
    "lib": [],
    "nofinal": [("    __syncthreads();\n    if (!am_last) return;", "    __syncthreads();\n    if (n >= 0) return;")],
    "upt4": [("constexpr int64_t kUnitsPerThreadSmall = 2;", "constexpr int64_t kUnitsPerThreadSmall = 4;")],
    "upt1": [("constexpr int64_t kUnitsPerThreadSmall = 2;", "constexpr int64_t kUnitsPerThreadSmall = 1;")],
    "tpb512": [("constexpr int kDotTPB = 256;", "constexpr int kDotTPB = 512;")],
}

TIMER = r'''
import os, sys, torch
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
dx = synth.torch_uniform(0, 0, 40 << 20, device=dev)
dy = synth.torch_uniform(1, 0, 40 << 20, device=dev)
for n in (1 << 20, 1 << 22, 1 << 24):
    copies = max(2, min(40, (300 << 20) // (8 * n)))
    res = torch.empty((), device=dev)
    calls = [(lambda k=k, n=n: lift.lift_dot(dx[k * n:(k + 1) * n], dy[k * n:(k + 1) * n], out=res)) for k in range(copies)]
    reps = max(20, copies)
    t = graph_time([calls[j % copies] for j in range(reps)])
    print(f"  n=2^{n.bit_length()-1:2d}: {t:7.2f} us  {8*n/t/1e3:7.1f} GB/s", flush=True)
'''


def patched(name):
    d = f"/tmp/dot_var_{name}"
    shutil.rmtree(d, ignore_errors=True)
    os.makedirs(d)
    for sub in ("paper_conf_cgo_steuwerrd17_b200", "include", "synth", "oracle", "tools"):
        shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                        ignore=shutil.ignore_patterns("_build", "*.so", "__pycache__"))
    shutil.copy(os.path.join(ROOT, "__graft_entry__.py"), d)
    src = open(SRC).read()
    for old, new in VARIANTS[name]:
        assert old in src, (name, old)
        src = src.replace(old, new)
    open(os.path.join(d, "paper_conf_cgo_steuwerrd17_b200", "csrc", "dot.cu"), "w").write(src)
    subprocess.run([sys.executable, "-c", "import __graft_entry__ as g; g.build()"], cwd=d, check=True)
    return d


for rep in range(2):
    for name in sys.argv[1:] or list(VARIANTS):
        d = patched(name) if rep == 0 else f"/tmp/dot_var_{name}"
        print(f"== {name}", flush=True)
        subprocess.run([sys.executable, "-c", TIMER], cwd=d, check=True)
