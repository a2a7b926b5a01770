"""Host-side cost per library call (tuning aid): wall time of N eager calls of
each op on tiny inputs (GPU work negligible), through the C ABI via ctypes, and
the same for an empty torch op as the floor of Python + launch overhead.
usage: python tools/host_overhead.py"""
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")
L = lift.lib()
s = torch.cuda.current_stream().cuda_stream
x = torch.rand(1024, device=dev)
A = torch.rand(64, 1024, device=dev)
y = torch.empty(64, device=dev)
r = torch.empty((), device=dev)
yt = torch.empty(1024, device=dev)
ws_dot = torch.zeros(L.lift_dot_workspace_bytes(1024), dtype=torch.uint8, device=dev)
ws_atax = torch.zeros(L.lift_atax_workspace_bytes(64, 1024), dtype=torch.uint8, device=dev)
calls = {
    "torch x.add_(0) (floor)": lambda: x.add_(0),
    "lift_dot C ABI": lambda: L.lift_dot(1024, x.data_ptr(), x.data_ptr(), r.data_ptr(), ws_dot.data_ptr(),
                                         ws_dot.numel(), s),
    "lift_gemv C ABI": lambda: L.lift_gemv(64, 1024, A.data_ptr(), x.data_ptr(), y.data_ptr(), s),
    "lift_atax C ABI": lambda: L.lift_atax(64, 1024, A.data_ptr(), x.data_ptr(), yt.data_ptr(), ws_atax.data_ptr(),
                                           ws_atax.numel(), s),
    "lift.lift_gemv (binding)": lambda: lift.lift_gemv(A, x, out=y),
    "lift.lift_dot (binding)": lambda: lift.lift_dot(x, x, out=r),
    "lift.lift_atax (binding)": lambda: lift.lift_atax(A, x, out=yt),
}
for name, fn in calls.items():
    for _ in range(200):
        fn()
    torch.cuda.synchronize()
    best = 1e9
    for _ in range(5):
        t0 = time.perf_counter()
        for _ in range(2000):
            fn()
        t1 = time.perf_counter()
        torch.cuda.synchronize()
        best = min(best, (t1 - t0) / 2000 * 1e6)
    print(f"{name:28s} {best:7.2f} us/call (host)", flush=True)
