"""A/B of the src-sorted bulk build (a3): one process per setting (env / DG_LIB_PATH).
Prints the insert call and kernel times of the sorted and random-order builds of cfg2.

    DG_EXCL_CHAINS=64 python tools/sorted_ab.py
"""
import json
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph  # noqa: E402


def build(nv, hints, s, d, w, reps=3):
    cu = lambda x: torch.from_numpy(np.ascontiguousarray(x)).cuda()  # noqa: E731
    S, D, W = cu(s), cu(d), cu(w)
    out = []
    for _ in range(reps):
        g = Graph(nv, hints)
        torch.cuda.synchronize()
        g.profile_enable(True)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        n = g.insert_edges(S, D, W, count=True)
        b.record()
        torch.cuda.synchronize()
        p = g.profile_read()
        out.append((a.elapsed_time(b), p["kernel_ms"]["insert"], n))
        inv = g.check_invariants()
        assert inv["violations"] == 0, inv
        g.close()
    return out


def main():
    cfg = bench.CONFIGS[os.environ.get("CFG", "cfg2")]
    nv, m, bs, bd, bw = bench.build_base(cfg)
    hints = torch.bincount(torch.from_numpy(bs.astype(np.int64)).cuda(), minlength=nv).to(torch.int32)
    order = np.argsort(bs, kind="stable")
    res = {"env": {k: v for k, v in os.environ.items() if k.startswith("DG_")},
           "random": build(nv, hints, bs, bd, bw),
           "sorted": build(nv, hints, bs[order], bd[order], bw[order])}
    print(json.dumps(res))


if __name__ == "__main__":
    main()
