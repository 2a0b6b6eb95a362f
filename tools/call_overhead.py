"""Per-call overhead of small batches: cfg2 graph, 2^B-op batches.
For insert / delete / query prints, per call: the bench-style device time of one call
between two events (Python binding + library host code + kernels), the device time
per call of 50 back-to-back calls, the library's kernel time (profile), and the host
time per call (Python + library)."""
import json
import os
import sys
import time

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402
import workloads as wl  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph  # noqa: E402


def main():
    B = 1 << int(os.environ.get("BLOG2", "16"))
    cfg = bench.CONFIGS["cfg2"]
    nv, m, bs, bd, bw = bench.build_base(cfg)
    dev = torch.device("cuda", 0)
    cu = lambda x: torch.from_numpy(np.ascontiguousarray(x)).to(dev)  # noqa: E731
    hints = torch.bincount(cu(bs.astype(np.int64)), minlength=nv).to(torch.int32)
    g = Graph(nv, hints)
    g.insert_edges(cu(bs), cu(bd), cu(bw), count=True)
    K = 50
    batches = [tuple(cu(x) for x in wl.uniform_edges(9, 100 + k, B, nv)) for k in range(K)]
    found = torch.empty(B, dtype=torch.uint8, device=dev)
    wout = torch.empty(B, dtype=torch.uint32, device=dev)
    ops = {"insert": lambda b: g.insert_edges(b[0], b[1], b[2]),
           "query": lambda b: g.query_edges(b[0], b[1], found_out=found, weight_out=wout),
           "delete": lambda b: g.delete_edges(b[0], b[1])}
    out = {"batch": B}
    for name, fn in ops.items():
        for b in batches[:3]:
            fn(b)
        torch.cuda.synchronize()
        # one call between events (the bench's measurement)
        single = []
        for b in batches[:10]:
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            torch.cuda.synchronize()
            e0.record()
            fn(b)
            e1.record()
            torch.cuda.synchronize()
            single.append(e0.elapsed_time(e1) * 1e3)
        # back to back (one untimed pass first: the pools reach their steady-state
        # headroom, before the timed pass)
        for b in batches:
            fn(b)
        torch.cuda.synchronize()
        g.profile_enable(True)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        t0 = time.perf_counter()
        for b in batches:
            fn(b)
        t1 = time.perf_counter()
        e1.record()
        torch.cuda.synchronize()
        p = g.profile_read()
        g.profile_enable(False)
        kind = name
        out[name] = {"single_call_us": float(np.median(single)),
                     "back_to_back_us": e0.elapsed_time(e1) * 1e3 / K,
                     "kernel_us": p["kernel_ms"][kind] * 1e3 / max(1, p["kernel_launches"][kind]),
                     "host_us": (t1 - t0) * 1e6 / K,
                     "launches_per_call": p["launches"] / K}
    print(json.dumps(out))


if __name__ == "__main__":
    main()
