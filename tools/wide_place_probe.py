import os, sys, torch
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
m, n = 8192, 32768
per = m * n
x = synth.torch_uniform(0, 0, n, device=dev); y = torch.empty(n, device=dev)
# (a) separate allocations
As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(2)]
print("separate  ", graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 12)[:12]]))
del As
# (b) one pool, views at k*per
for extra in (0, 1 << 20, 3 << 20):
    pool = synth.torch_uniform(2, 0, 2 * per + extra, device=dev)
    As = [pool[extra + k * per: extra + (k + 1) * per].view(m, n) for k in range(2)]
    print("pool off", extra, graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 12)[:12]]))
    del pool, As
# (c) x inside the pool tail like table1
pool = synth.torch_uniform(2, 0, 3 * per, device=dev)
As = [pool[k * per:(k + 1) * per].view(m, n) for k in range(2)]
xp = pool[-n:]
print("pool + x in pool", graph_time([(lambda A=A: lift.lift_atax(A, xp, out=y, algo="fused")) for A in (As * 12)[:12]]))
print("pool + x separate", graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 12)[:12]]))
