"""Profiling driver (ncu target): builds a config graph with degree hints, then runs
a src-sorted bulk build (second graph) and one bench step (insert / query / delete of
2^B edges) so `ncu -k regex:... -c N` can capture each kernel once.

    ncu --set full -k regex:k_edges -c 3 python tools/prof_cfg.py --config cfg2
"""
import argparse
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402
import workloads as wl  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="cfg2")
    ap.add_argument("--batch-log2", type=int, default=24)
    ap.add_argument("--bucket-bytes", type=int, default=128)
    ap.add_argument("--no-sorted", action="store_true")
    a = ap.parse_args()
    cfg = bench.CONFIGS[a.config]
    dev = torch.device("cuda", 0)
    nv, m, bs, bd, bw = bench.build_base(cfg)
    hints = torch.bincount(torch.from_numpy(bs.astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
    cu = lambda x: torch.from_numpy(np.ascontiguousarray(x)).to(dev)  # noqa: E731
    g = Graph(nv, hints, bucket_bytes=a.bucket_bytes)
    g.insert_edges(cu(bs), cu(bd), cu(bw), count=True)  # random-order bulk build
    if not a.no_sorted:
        order = np.argsort(bs, kind="stable")
        g2 = Graph(nv, hints, bucket_bytes=a.bucket_bytes)
        g2.insert_edges(cu(bs[order]), cu(bd[order]), cu(bw[order]), count=True)
        g2.close()
    B = 1 << a.batch_log2
    (s, d, w), (qs, qd), (xs, xd) = bench.step_batch(cfg, nv, B, 0, 0, 1, (None, m, (bs, bd)))
    g.insert_edges(cu(s), cu(d), cu(w))
    g.query_edges(cu(qs), cu(qd))
    g.delete_edges(cu(xs), cu(xd))
    torch.cuda.synchronize()
    g.close()
    print("prof_cfg done", a.config)


if __name__ == "__main__":
    main()
