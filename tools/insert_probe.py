"""Quick insert-path timing on cfg2 (bulk build + one random insert/delete round).
Used for kernel tuning under ncu; not part of the bench contract."""
import sys, os, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph

nv, m = 4_847_571, 68_993_773
rounds = int(sys.argv[1]) if len(sys.argv) > 1 else 2
reuse = os.environ.get("REUSE", "1") == "1"
s, d = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
w = wl.weights(2, 0, m)
dev = torch.device("cuda", 0)
hints = torch.bincount(torch.from_numpy(s.astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
S, D, Wt = (torch.from_numpy(x).to(dev) for x in (s, d, w))
g = Graph(nv, hints, reuse_tombstones=reuse)
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
torch.cuda.synchronize()
e0.record(); n = g.insert_edges(S, D, Wt, count=True); e1.record(); torch.cuda.synchronize()
print(f"bulk insert {e0.elapsed_time(e1):.2f} ms added {n}", g.stats())
B = 1 << 24
for r in range(rounds):
    bs, bd, bw = wl.uniform_edges(2, 1000 + r, B, nv)
    BS, BD, BW = (torch.from_numpy(x).to(dev) for x in (bs, bd, bw))
    torch.cuda.synchronize()
    e0.record(); n = g.insert_edges(BS, BD, BW, count=True); e1.record(); torch.cuda.synchronize()
    ti = e0.elapsed_time(e1)
    e0.record(); k = g.delete_edges(BS, BD, count=True); e1.record(); torch.cuda.synchronize()
    print(f"round {r}: insert {ti:.2f} ms ({n}) delete {e0.elapsed_time(e1):.2f} ms ({k})")
print(g.stats())
