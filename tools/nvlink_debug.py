import os, sys, time, subprocess
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def child(world, n, offs, sleep):
    import synth
    from paper_conf_cgo_steuwerrd17_b200 import nvlink
    dev = torch.device("cuda:0")
    x = synth.torch_uniform(0, 0, n + 8, device=dev)
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, world, dev)
    ws = [torch.zeros(nvlink.workspace_bytes("dot", 0, n), dtype=torch.uint8, device=dev) for _ in range(world)]
    res = [torch.empty((), device=dev) for _ in range(world)]
    s = [torch.cuda.Stream() for _ in range(world)]
    per = n // world
    torch.cuda.synchronize()
    t0 = time.time()
    for r in range(world):
        a = offs[r] + r * per
        with torch.cuda.stream(s[r]):
            nvlink.lift_dot_allreduce(x[a:a + per], x[a:a + per], exs[r], out=res[r], workspace=ws[r])
        if sleep:
            time.sleep(0.2)
    torch.cuda.synchronize()
    print("ok", [round(v.item(), 2) for v in res], round(time.time() - t0, 3))


if len(sys.argv) > 1:
    a = sys.argv[1:]
    child(int(a[0]), int(a[1]), [int(v) for v in a[2].split(",")], int(a[3]))
    sys.exit(0)
cases = [(1, 1 << 20, "0", 0), (1, 1 << 20, "1", 0), (2, 1 << 20, "0,0", 0), (2, 1 << 20, "1,1", 0),
         (2, 1 << 20, "0,1", 0), (2, 1 << 20, "0,1", 1), (2, 1 << 16, "0,0", 0), (2, 1 << 16, "0,1", 0),
         (2, 4096, "1,1", 0)]
for c in cases:
    r = subprocess.run([sys.executable, __file__, str(c[0]), str(c[1]), c[2], str(c[3])], capture_output=True, text=True,
                       timeout=60)
    out = (r.stdout.strip().splitlines() or ["?"])[-1]
    print(c, "->", out if r.returncode == 0 else "FAIL " + (r.stderr.strip().splitlines() or ["?"])[-1][:60], flush=True)
