"""Quick per-op timing probe (CUDA events, L2 flushed between iterations).
Not the bench contract (bench.py); used while tuning."""
import json
import sys
import time

import torch

sys.path.insert(0, __import__("os").path.dirname(__import__("os").path.dirname(__import__("os").path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402


def timeit(fn, iters=20, flush=None):
    if QUICK:
        iters = 2
    ts = []
    for i in range(iters + 3):
        if flush is not None:
            flush.sum()  # read-only flush: L2 left holding clean lines of another buffer
        s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s.record()
        fn()
        e.record()
        e.synchronize()
        if i >= 3:
            ts.append(s.elapsed_time(e) * 1e3)
    ts.sort()
    return ts[len(ts) // 2], ts[0]


QUICK = "--quick" in sys.argv


def main():
    dev = torch.device("cuda:0")
    props = torch.cuda.get_device_properties(dev)
    print(json.dumps({"gpu": props.name, "sms": props.multi_processor_count, "l2": getattr(props, "L2_cache_size", None)}))
    flush = torch.ones(128 << 20, dtype=torch.float32, device=dev)
    res = []

    def rep(name, nbytes, fn, **kw):
        med, mn = timeit(fn, flush=flush)
        res.append((name, med, mn, nbytes / med / 1e3))
        print(f"{name:40s} med {med:9.2f} us  min {mn:9.2f} us  {nbytes / med / 1e3:8.1f} GB/s  {nbytes/mn/1e3:8.1f} GB/s(min)", flush=True)

    # pure read probe: torch sum as a reference point
    n = 1 << 28
    big = torch.empty(n, device=dev).fill_(1.0)
    rep("torch.sum 1 GiB", n * 4, lambda: big.sum())
    rep("torch copy 1 GiB (r+w)", n * 8, lambda: big.clone())
    del big
    for n in (1 << 20, 1 << 24, 1 << 26, 1 << 28, 1 << 30):
        x = synth.torch_uniform(0, 0, n, device=dev)
        y = synth.torch_uniform(1, 0, n, device=dev)
        rep(f"dot n={n}", 8 * n, lambda: lift.lift_dot(x, y))
        del x, y
    for m, n in ((4096, 4096), (8192, 8192), (65536, 32768)):
        A = synth.torch_matrix_rows(2, n, 0, m, device=dev)
        x = synth.torch_uniform(0, 0, n, device=dev)
        y = torch.empty(m, device=dev)
        rep(f"gemv {m}x{n}", 4 * m * n + 4 * (m + n), lambda: lift.lift_gemv(A, x, out=y))
        if m <= 8192 and not QUICK:
            for wpr, rg in ((8, 1), (8, 2), (4, 2), (4, 4), (2, 4), (2, 8), (1, 8)):
                for xs in (0, 1):
                    rep(f"  gemv tuned wpr={wpr} rg={rg} xs={xs}", 4 * m * n, lambda: lift.lift_gemv_tuned(A, x, out=y, wpr=wpr, rg=rg, xsmem=xs))
        if m == 8192:
            B = synth.torch_matrix_rows(3, n, 0, m, device=dev)
            rep(f"gesummv {m}x{n}", 8 * m * n + 4 * (m + n), lambda: lift.lift_gesummv(1.5, A, 1.2, B, x, out=y))
            for wpr, rg in (() if QUICK else ((8, 1), (4, 2), (2, 4), (1, 8))):
                rep(f"  gesummv tuned wpr={wpr} rg={rg}", 8 * m * n, lambda: lift.lift_gesummv_tuned(1.5, A, 1.2, B, x, out=y, wpr=wpr, rg=rg))
            del B
            yy = torch.empty(n, device=dev)
            rep(f"atax fused {m}x{n}", 4 * m * n, lambda: lift.lift_atax(A, x, out=yy, algo="fused"))
            rep(f"atax twopass {m}x{n} (8mn bytes)", 8 * m * n, lambda: lift.lift_atax(A, x, out=yy, algo="twopass"))
        if m == 4096:
            yy = torch.empty(n, device=dev)
            rep(f"atax fused {m}x{n}", 4 * m * n, lambda: lift.lift_atax(A, x, out=yy, algo="fused"))
            rep(f"atax twopass {m}x{n} (8mn bytes)", 8 * m * n, lambda: lift.lift_atax(A, x, out=yy, algo="twopass"))
        del A


if __name__ == "__main__":
    main()
