"""Incremental build without degree hints (Tab. VI geometry: 1 bucket per vertex) on
the cfg2 R-MAT: batches of 2^22 edges; reports per-batch insert time and chain stats."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
nv, m = 4_847_571, 68_993_773
s, d = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
w = wl.weights(2, 0, m)
dev = torch.device("cuda", 0)
S, D, W = (torch.from_numpy(x).to(dev) for x in (s, d, w))
for hints in (False, True):
    h = torch.bincount(S.to(torch.int64), minlength=nv).to(torch.int32) if hints else None
    g = Graph(nv, h)
    B = 1 << 22
    ev = lambda: torch.cuda.Event(enable_timing=True)
    tot = 0.0
    times = []
    for k in range(0, m, B):
        a, b = ev(), ev()
        torch.cuda.synchronize(); a.record()
        g.insert_edges(S[k:k + B], D[k:k + B], W[k:k + B])
        b.record(); torch.cuda.synchronize()
        times.append(a.elapsed_time(b))
    st = g.stats()
    print(f"hints={hints}: total {sum(times):.1f} ms ({m / sum(times) / 1e3:.0f} M edges/s), first/last batch "
          f"{times[0]:.2f}/{times[-1]:.2f} ms, max_chain {st['max_chain']}, overflow {st['overflow_buckets']}, "
          f"lf {st['load_factor']:.3f}")
    q = g.query_edges(S[:B], D[:B])
    a, b = ev(), ev(); torch.cuda.synchronize(); a.record(); g.query_edges(S[:B], D[:B]); b.record(); torch.cuda.synchronize()
    print(f"   query 2^22 live edges: {a.elapsed_time(b):.2f} ms")
    g.close()
