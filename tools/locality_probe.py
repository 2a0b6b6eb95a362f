"""Batch-order experiment: kernel time of the cfg2 step ops when the batch is
reordered for memory locality before the call (the reorder itself is NOT timed here:
this measures what a locality-ordered probe could gain, to decide whether an in-library
partition pass pays).  Orders: the generator's (uniform random), sources bucketed by
src >> k (stable, so the batch order of equal keys is kept), fully src-sorted.

    python tools/locality_probe.py [--config cfg2] [--reps 5]
"""
import argparse
import json
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="cfg2")
    ap.add_argument("--batch-log2", type=int, default=24)
    ap.add_argument("--reps", type=int, default=5)
    a = ap.parse_args()
    cfg = bench.CONFIGS[a.config]
    dev = torch.device("cuda", 0)
    nv, m, bs, bd, bw = bench.build_base(cfg)
    hints = torch.bincount(torch.from_numpy(bs.astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
    cu = lambda x: torch.from_numpy(np.ascontiguousarray(x)).to(dev)  # noqa: E731
    g = Graph(nv, hints)
    g.insert_edges(cu(bs), cu(bd), cu(bw), count=True)
    B = 1 << a.batch_log2
    flush = torch.empty(256 << 20, dtype=torch.uint8, device=dev)
    found = torch.empty(B, dtype=torch.uint8, device=dev)
    qw = torch.empty(B, dtype=torch.int32, device=dev)
    out = {}
    shift_bits = int(np.ceil(np.log2(nv)))
    for order in ["random", "k16", "k12", "k8", "k4", "sorted"]:
        res = {"insert": [], "query": [], "delete": []}
        for rep in range(a.reps):
            (s, d, w), (qs, qd), (xs, xd) = bench.step_batch(cfg, nv, B, rep, 0, 1, (None, m, (bs, bd)))
            S, D, W, QS, QD, XS, XD = (cu(x) for x in (s, d, w, qs, qd, xs, xd))
            if order != "random":
                k = 0 if order == "sorted" else int(order[1:])
                def perm(x):
                    key = x.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
                    return torch.sort(key >> k, stable=True).indices

                def take(x, p):  # (no uint32 gather kernels in torch)
                    return x.view(torch.int32)[p].view(x.dtype)
                p = perm(S); S, D, W = take(S, p), take(D, p), take(W, p)
                p = perm(QS); QS, QD = take(QS, p), take(QD, p)
                p = perm(XS); XS, XD = take(XS, p), take(XD, p)
            torch.cuda.synchronize()
            g.profile_enable(True)
            p0 = g.profile_read()
            flush.zero_()
            g.insert_edges(S, D, W)
            flush.zero_()
            g.query_edges(QS, QD, found_out=found, weight_out=qw)
            flush.zero_()
            g.delete_edges(XS, XD)
            torch.cuda.synchronize()
            p1 = g.profile_read()
            g.profile_enable(False)
            g.delete_edges(cu(s), cu(d))  # back to the base graph
            torch.cuda.synchronize()
            if rep == 0:
                continue  # warm-up
            for op in res:
                res[op].append(p1["kernel_ms"][op] - p0["kernel_ms"][op])
        out[order] = {op: round(float(np.median(v)), 4) for op, v in res.items()}
        print(order, out[order], flush=True)
    print(json.dumps({"config": a.config, "batch": B, "nv": nv, "shift_bits": shift_bits,
                      "kernel_ms_median": out}))
    g.close()


if __name__ == "__main__":
    main()
