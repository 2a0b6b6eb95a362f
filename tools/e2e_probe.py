"""Breakdown of the host-buffer (e2e) path: per call wall time vs raw H2D/D2H copy time."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
nv, B = 4_847_571, 1 << 24
dev = torch.device("cuda", 0)
g = Graph(nv, np.full(nv, 14, np.uint32))
s, d, w = wl.uniform_edges(2, 1, B, nv)
hs, hd, hw = (torch.from_numpy(x).pin_memory() for x in (s, d, w))
hf = torch.empty(B, dtype=torch.uint8).pin_memory()
hq = torch.empty(B, dtype=torch.uint32).pin_memory()
dst = torch.empty(B, dtype=torch.uint32, device=dev)
for rep in range(3):
    torch.cuda.synchronize()
    t0 = time.perf_counter(); dst.copy_(hs, non_blocking=True); torch.cuda.synchronize(); t1 = time.perf_counter()
    hq.copy_(dst, non_blocking=True); torch.cuda.synchronize(); t2 = time.perf_counter()
    g.insert_edges(hs, hd, hw); t3 = time.perf_counter()
    g.query_edges(hs, hd, found_out=hf, weight_out=hq); t4 = time.perf_counter()
    g.delete_edges(hs, hd); t5 = time.perf_counter(); torch.cuda.synchronize(); t6 = time.perf_counter()
    print(f"H2D 64MB {1e3*(t1-t0):.2f} ms ({64/(t1-t0)/1e3:.1f} GB/s)  D2H 64MB {1e3*(t2-t1):.2f} ms  "
          f"insert {1e3*(t3-t2):.2f}  query {1e3*(t4-t3):.2f}  delete {1e3*(t5-t4):.2f} ms  (+{1e3*(t6-t5):.2f} kernel tail)  step {1e3*(t6-t2):.2f} ms")
