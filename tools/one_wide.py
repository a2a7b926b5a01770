import os, sys, torch
sys.path.insert(0, os.getcwd())
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift
dev = torch.device("cuda:0")
m, n = 8192, 32768
A = synth.torch_matrix_rows(2, n, 0, m, device=dev); x = synth.torch_uniform(0, 0, n, device=dev)
for _ in range(3): y = lift.lift_atax(A, x, algo="fused")
torch.cuda.synchronize()
