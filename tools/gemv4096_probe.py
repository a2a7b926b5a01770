"""Where GEMV 4096^2's time goes (tuning aid).  Runs the library's GEMV at
4096 x 4096 under several launch configurations (lift_gemv_tuned) next to a
pure 64 MiB streaming read (lift_dot over two 32 MiB vectors: the same bytes,
no x, no per-row reduction).

  python tools/gemv4096_probe.py time   CUDA-graph timing (24 calls per graph,
                                        operands rotated past L2), best of 3
  python tools/gemv4096_probe.py ncu    each variant launched 3x (run under
                                        ncu --metrics ...; the last launch of
                                        each is the one to read)
"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
# LIFT_ROOT: the package root to time (tools/ab_tree.sh points it at an older tree)
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

mode = sys.argv[1] if len(sys.argv) > 1 else "time"
dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
m = n = 4096
sets = max(2, -(-3 * L2 // (4 * m * n)))
As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
x = synth.torch_uniform(0, 0, n, device=dev)
y = torch.empty(m, device=dev)
half = m * n // 2
xs = [synth.torch_uniform(50 + k, 0, half, device=dev) for k in range(sets)]
ys = [synth.torch_uniform(70 + k, 0, half, device=dev) for k in range(sets)]
r = torch.empty((), device=dev)

VARIANTS = {
    "gemv auto": lambda A: lift.lift_gemv(A, x, out=y),
    "gemv wpr8 rg1 lb8": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=8, rg=1, lb=8),
    "gemv wpr8 rg2": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=8, rg=2),
    "gemv wpr4 rg2": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=4, rg=2),
    "gemv wpr4 rg4": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=4, rg=4),
    "gemv wpr2 rg4": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=2, rg=4),
    "gemv wpr1 rg8": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=1, rg=8),
    "gemv wpr1 rg8 lb8": lambda A: lift.lift_gemv_tuned(A, x, out=y, wpr=1, rg=8, lb=8),
    "gemv xsmem0": lambda A: lift.lift_gemv_tuned(A, x, out=y, xsmem=0),
    "gemv blocks296": lambda A: lift.lift_gemv_tuned(A, x, out=y, blocks=296),
    "gemv blocks1184": lambda A: lift.lift_gemv_tuned(A, x, out=y, blocks=1184),
}
tiny_A = torch.ones(1, 4, device=dev)
tiny_x = torch.ones(4, device=dev)
tiny_y = torch.empty(1, device=dev)
if mode == "ncu":
    for k in range(3):  # the launch floor: a 1 x 4 GEMV (one block, no traffic)
        lift.lift_gemv(tiny_A, tiny_x, out=tiny_y)
    torch.cuda.synchronize()
    for name, f in VARIANTS.items():
        for k in range(3):
            f(As[k % sets])
        torch.cuda.synchronize()
    for k in range(3):
        lift.lift_dot(xs[k % sets], ys[k % sets], out=r)
    torch.cuda.synchronize()
else:
    from sweep import graph_time

    for name, f in VARIANTS.items():
        t = graph_time([(lambda A=A: f(A)) for A in (As * 24)[:24]])
        print(f"{name:22s} {t:7.2f} us  {4 * m * n / t / 1e3:7.1f} GB/s", flush=True)
    t = graph_time([(lambda k=k: lift.lift_dot(xs[k % sets], ys[k % sets], out=r)) for k in range(24)])
    print(f"{'dot 2x32MiB (read)':22s} {t:7.2f} us  {4 * m * n / t / 1e3:7.1f} GB/s", flush=True)
