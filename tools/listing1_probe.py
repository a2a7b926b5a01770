"""Launch-shape probe for the Listing-1 kernel (NEXT-3), tuning aid.

Builds patched copies of the package under /tmp with other values of
listing1.cu's kL1Unroll / kL1Pipe / kL1BlocksPerSm (the library is not
changed) and times lift_partial_dot and lift_dot_listing1 at 2^20 and 2^28
(CUDA graph of back-to-back calls on distinct slices, > 2x L2), next to
k_dot at the same sizes.  Every variant is checked bitwise against the
library's result first.
usage: SIZES=20,28 python tools/listing1_probe.py [unroll,pipe,blocks_per_sm ...]
"""
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PKG = "paper_conf_cgo_steuwerrd17_b200"
VARIANTS = [tuple(int(a) if a.isdigit() else a for a in v.split(",")) for v in sys.argv[1:]] or [
    (4, "false", 8), (4, "false", 5), (2, "true", 8), (4, "true", 8), (4, "true", 4), (8, "false", 8),
    (2, "false", 8), (8, "true", 8)]
SIZES = os.environ.get("SIZES", "20,28")

TIMER = r'''
import os, sys
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import torch, synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
tag = os.environ["VARIANT"]
x = synth.torch_uniform(0, 0, 1 << 29, device=dev)
y = synth.torch_uniform(1, 0, 1 << 29, device=dev)
ref = torch.load(os.environ["REF"]) if os.path.exists(os.environ["REF"]) else None
got = lift.lift_partial_dot(x[:1 << 22], y[:1 << 22])
if ref is None:
    torch.save(got.cpu(), os.environ["REF"])
else:
    assert torch.equal(got.cpu(), ref), tag
for n in [1 << int(e) for e in os.environ["SIZES"].split(",")]:
    copies = int(-(-2 * l2 // (8 * n))) + 1
    z = torch.empty(n // 128, device=dev)
    r = torch.empty((), device=dev)
    sl = [(x[k * n:(k + 1) * n], y[k * n:(k + 1) * n]) for k in range(copies)]
    reps = max(20, copies)
    for name, fn in (("partial_dot", lambda a, b: lift.lift_partial_dot(a, b, out=z)),
                     ("dot_listing1", lambda a, b: lift.lift_dot_listing1(a, b, out=r)),
                     ("k_dot", lambda a, b: lift.lift_dot(a, b, out=r))):
        if name == "k_dot" and tag != "library":
            continue
        t = graph_time([(lambda a=a, b=b, fn=fn: fn(a, b)) for a, b in (sl * reps)[:reps]])
        print(f"{tag:28s} {name:13s} n=2^{n.bit_length() - 1}: {t:9.2f} us  {8 * n / t / 1e3:8.1f} GB/s", flush=True)
'''


def patched(unroll, pipe, bps) -> str:
    d = f"/tmp/l1_{unroll}_{pipe}_{bps}"
    shutil.rmtree(d, ignore_errors=True)
    os.makedirs(d)
    for sub in (PKG, "include", "synth", "tools"):
        shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                        ignore=shutil.ignore_patterns("_build", "*.so", "__pycache__"))
    f = os.path.join(d, PKG, "csrc", "listing1.cu")
    s = open(f).read()
    for old, new in (("constexpr int kL1Unroll = 4;", f"constexpr int kL1Unroll = {unroll};"),
                     ("constexpr bool kL1Pipe = false;", f"constexpr bool kL1Pipe = {pipe};"),
                     ("constexpr int kL1BlocksPerSm = 8;", f"constexpr int kL1BlocksPerSm = {bps};")):
        assert old in s, old
        s = s.replace(old, new)
    open(f, "w").write(s)
    subprocess.run([sys.executable, "-c", f"import sys; sys.path.insert(0, '{d}'); from {PKG} import build; "
                    "build.build(force=True)"], check=True, cwd=d)
    return d


REF = "/tmp/l1_ref.pt"
if os.path.exists(REF):
    os.remove(REF)
subprocess.run([sys.executable, "-c", TIMER], cwd=ROOT, check=True, env=dict(os.environ, VARIANT="library", REF=REF, SIZES=SIZES))
for v in VARIANTS:
    d = patched(*v)
    subprocess.run([sys.executable, "-c", TIMER], cwd=d, check=True,
                   env=dict(os.environ, VARIANT=f"unroll {v[0]} pipe {v[1]} bps {v[2]}", REF=REF, SIZES=SIZES))
