"""TC timing at R-MAT scale s (symmetrised), cfg5-style dynamic iterations:
python tools/tc_probe.py [scale] [bucket_bytes] [map|set] [iters]"""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import workloads as wl
from paper_conf_ipps_awadapo20_b200 import Graph
scale = int(sys.argv[1]) if len(sys.argv) > 1 else 22
bb = int(sys.argv[2]) if len(sys.argv) > 2 else 128
var = sys.argv[3] if len(sys.argv) > 3 else "set"
iters = int(sys.argv[4]) if len(sys.argv) > 4 else 2
nv = 1 << scale
s, d = wl.rmat_edges(5, 0, 16 * nv, scale, wl.GRAPH500)
dev = torch.device("cuda", 0)
deg = torch.bincount(torch.from_numpy(np.concatenate([s, d]).astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
g = Graph(nv, deg, directed=False, bucket_bytes=bb, set_variant=var == "set")
g.insert_edges(torch.from_numpy(s).to(dev), torch.from_numpy(d).to(dev))
g.profile_enable(True)
prev = 0.0
for r in range(iters):
    if r:
        s1, d1 = wl.rmat_edges(5, r, 1 << 22, scale, wl.GRAPH500)
        g.insert_edges(torch.from_numpy(s1).to(dev), torch.from_numpy(d1).to(dev))
    torch.cuda.synchronize(); t0 = time.perf_counter()
    c = g.triangle_count()
    t1 = time.perf_counter()
    p = g.profile_read()
    st = g.stats()
    print(f"scale {scale} S={bb} {var} iter {r}: triangles {c}  total {1e3*(t1-t0):.1f} ms  wedge kernel "
          f"{p['kernel_ms']['tc'] - prev:.1f} ms  max_chain {st['max_chain']} lf {st['load_factor']:.3f}", flush=True)
    prev = p['kernel_ms']['tc']
