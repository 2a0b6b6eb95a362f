"""Bulk build on the cfg2 R-MAT with exact degree hints: wall time of
dg_create and of the single insert batch vs the insert kernel's device time, three
times in one process (first-touch / allocation effects vs steady state)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
nv, m = 4_847_571, 68_993_773
s, d = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
w = wl.weights(2, 0, m)
dev = torch.device("cuda", 0)
S, D, W = (torch.from_numpy(x).to(dev) for x in (s, d, w))
h = torch.bincount(S.to(torch.int64), minlength=nv).to(torch.int32)
order = torch.argsort(S.to(torch.int64))
Ss, Ds, Ws = (x.view(torch.int32)[order].view(torch.uint32).contiguous() for x in (S, D, W))
for it in range(4):
    srt = it == 3
    torch.cuda.synchronize(); t0 = time.perf_counter()
    g = Graph(nv, h)
    torch.cuda.synchronize(); t1 = time.perf_counter()
    g.profile_enable(True)
    n = g.insert_edges(Ss if srt else S, Ds if srt else D, Ws if srt else W, count=True)
    torch.cuda.synchronize(); t2 = time.perf_counter()
    p = g.profile_read()
    st = g.stats()
    print(f"iter {it}{' (src-sorted)' if srt else ''}: create {1e3*(t1-t0):.1f} ms, insert wall {1e3*(t2-t1):.1f} ms, "
          f"kernel {p['kernel_ms']['insert']:.2f} ms over {p['kernel_launches']['insert']} launches, added {n}, "
          f"overflow {st['overflow_buckets']}, max_chain {st['max_chain']}", flush=True)
    g.close()
