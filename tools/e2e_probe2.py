"""e2e host-call breakdown with fresh pinned buffers per step (as bench.py does) vs reused."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
nv, B = 4_847_571, 1 << 24
g = Graph(nv, np.full(nv, 14, np.uint32))
def pin(x): return torch.from_numpy(np.ascontiguousarray(x)).pin_memory()
for mode in ("fresh", "fresh", "reuse", "reuse", "fresh-touched", "fresh-touched"):
    if mode.startswith("fresh") or mode == "reuse" and "hs" not in globals():
        s, d, w = wl.uniform_edges(2, 1, B, nv)
        qs, qd, _ = wl.uniform_edges(2, 2, B, nv)
        hs, hd, hw, hq, hqd = (pin(x) for x in (s, d, w, qs, qd))
        hf = torch.empty(B, dtype=torch.uint8).pin_memory()
        hqw = torch.empty(B, dtype=torch.uint32).pin_memory()
        if mode == "fresh-touched":
            hf.fill_(0); hqw.fill_(0)
    torch.cuda.synchronize()
    t0 = time.perf_counter(); g.insert_edges(hs, hd, hw)
    t1 = time.perf_counter(); g.query_edges(hq, hqd, found_out=hf, weight_out=hqw)
    t2 = time.perf_counter(); g.delete_edges(hs, hd)
    t3 = time.perf_counter(); torch.cuda.synchronize(); t4 = time.perf_counter()
    print(f"{mode:14s} insert {1e3*(t1-t0):.2f}  query {1e3*(t2-t1):.2f}  delete {1e3*(t3-t2):.2f}  tail {1e3*(t4-t3):.2f}  step {1e3*(t4-t0):.2f} ms", flush=True)
