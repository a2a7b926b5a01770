"""Per-step host cost of the Python binding (tuning aid).  usage: python tools/binding_profile.py"""
import os, sys, time, torch
sys.path.insert(0, os.getcwd())
import paper_conf_cgo_steuwerrd17_b200 as lift
from paper_conf_cgo_steuwerrd17_b200 import _check_tensor, _same_device, _stream, _on
dev = torch.device("cuda:0")
A = torch.rand(64, 1024, device=dev); x = torch.rand(1024, device=dev); y = torch.empty(64, device=dev)
def t(name, fn, N=20000):
    for _ in range(1000): fn()
    t0 = time.perf_counter()
    for _ in range(N): fn()
    print(f"{name:40s} {(time.perf_counter()-t0)/N*1e6:7.3f} us")
t("_check_tensor", lambda: _check_tensor(A, "A", 2))
t("_same_device", lambda: _same_device(A, x))
t("_stream", lambda: _stream(dev))
t("torch.cuda.current_stream().cuda_stream", lambda: torch.cuda.current_stream().cuda_stream)
t("torch.cuda.current_stream(dev)", lambda: torch.cuda.current_stream(dev))
t("_on(dev) enter/exit", lambda: _on(dev).__enter__())
t("torch.cuda.current_device()", lambda: torch.cuda.current_device())
t("A.data_ptr()", lambda: A.data_ptr())
t("A.shape unpack", lambda: tuple(A.shape))
t("lift.lib()", lambda: lift.lib())
t("torch.cuda.is_current_stream_capturing()", lambda: torch.cuda.is_current_stream_capturing())
t("torch._C._cuda_getCurrentRawStream(0)", lambda: torch._C._cuda_getCurrentRawStream(0))
