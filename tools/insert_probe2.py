"""Per-call host/device timing of the cfg2 bench sequence (insert / query / delete of
2^24 uniform edges, count=False), with DG_DEBUG pool-growth messages.  Diagnostic."""
import sys, os, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph

adaptive = os.environ.get("ADAPTIVE", "0") == "1"
if os.environ.get("CFG", "cfg2") == "cfg3":
    s, d = wl.grid_edges(3, 4894, 4894, 0.6025)
    nv, m = 4894 * 4894, s.size
else:
    nv, m = 4_847_571, 68_993_773
    s, d = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
w = wl.weights(2, 0, m)
dev = torch.device("cuda", 0)
hints = torch.bincount(torch.from_numpy(s.astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
S, D, Wt = (torch.from_numpy(x).to(dev) for x in (s, d, w))
g = Graph(nv, hints, adaptive=adaptive)
g.insert_edges(S, D, Wt)
torch.cuda.synchronize()
print(g.stats(), flush=True)
B = 1 << 24
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
for r in range(4):
    bs, bd, bw = wl.uniform_edges(2, 1000 + r, B, nv)
    BS, BD, BW = (torch.from_numpy(x).to(dev) for x in (bs, bd, bw))
    torch.cuda.synchronize()
    for name, fn in (("insert", lambda: g.insert_edges(BS, BD, BW)),
                     ("query", lambda: g.query_edges(BS, BD)),
                     ("delete", lambda: g.delete_edges(BS, BD))):
        t0 = time.perf_counter(); e0.record(); fn(); e1.record(); t1 = time.perf_counter()
        torch.cuda.synchronize()
        print(f"round {r} {name}: device {e0.elapsed_time(e1):.3f} ms host {1e3*(t1-t0):.3f} ms", flush=True)
print(g.stats())
