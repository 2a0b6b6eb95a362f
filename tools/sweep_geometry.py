"""Config-3 geometry sweep (SURVEY §8(d) cfg 3; Fig. 2 / Tab. VI questions):
road-like grid 4,894^2, load factor x bucket bytes x {hints, no hints (1 bucket per
vertex, the incremental-build geometry of Tab. VI)}.  For each point: bulk-build
time, insert / delete rate of 2^22 uniform random edges, memory and chain stats, and
an export digest (identical across every point = geometry invariance).

    python tools/sweep_geometry.py [out.json] [--quick]
"""
import hashlib
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import workloads as wl  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph  # noqa: E402


def digest(g):
    ro, d, w = g.export()
    lens = (ro[1:].to(torch.int64) - ro[:-1].to(torch.int64))
    rows = torch.repeat_interleave(torch.arange(lens.numel(), device=ro.device), lens)
    key = (rows << 32) | d.to(torch.int64)
    order = torch.argsort(key)
    k = key[order].cpu().numpy().tobytes()
    ww = w.to(torch.int64)[order].cpu().numpy().tobytes()
    return hashlib.sha256(k + ww).hexdigest()[:16]


def main():
    out = sys.argv[1] if len(sys.argv) > 1 and not sys.argv[1].startswith("--") else None
    quick = "--quick" in sys.argv
    dev = torch.device("cuda", 0)
    rows_, cols = (1024, 1024) if quick else (4894, 4894)
    bs, bd = wl.grid_edges(3, rows_, cols, 0.6025)
    nv = rows_ * cols
    # deterministic weights: equal keys carry equal weights, so exports must match bit for bit
    bw = (bs.astype(np.uint64) * 2654435761 ^ bd.astype(np.uint64)).astype(np.uint32)
    hints = torch.bincount(torch.from_numpy(bs.astype(np.int64)).to(dev), minlength=nv).to(torch.int32)
    BS, BD, BW = (torch.from_numpy(x).to(dev) for x in (bs, bd, bw))
    B = 1 << 22
    s, d, _ = wl.uniform_edges(3, 1000, B, nv)
    w = (s.astype(np.uint64) * 2654435761 ^ d.astype(np.uint64)).astype(np.uint32)
    S, D, Wt = (torch.from_numpy(x).to(dev) for x in (s, d, w))
    ev = lambda: torch.cuda.Event(enable_timing=True)  # noqa: E731
    res = []
    for bb in (32, 64, 128):
        for lf in (0.35, 0.5, 0.7, 1.0, 2.0, 5.0):
            for h in (True, False):
                torch.cuda.synchronize()
                e = [ev() for _ in range(6)]
                e[0].record()
                g = Graph(nv, hints if h else None, bucket_bytes=bb, load_factor=lf)
                e[1].record()
                g.insert_edges(BS, BD, BW)
                e[2].record()
                torch.cuda.synchronize()
                st_build = g.stats()
                e[3].record()
                g.insert_edges(S, D, Wt)
                e[4].record()
                g.delete_edges(S, D)
                e[5].record()
                torch.cuda.synchronize()
                st = g.stats()
                pt = {"bucket_bytes": bb, "load_factor": lf, "hints": h,
                      "create_ms": e[0].elapsed_time(e[1]), "bulk_insert_ms": e[1].elapsed_time(e[2]),
                      "bulk_M_edges_s": bs.size / (e[1].elapsed_time(e[2]) * 1e3),
                      "insert_M_edges_s": B / (e[3].elapsed_time(e[4]) * 1e3),
                      "delete_M_edges_s": B / (e[4].elapsed_time(e[5]) * 1e3),
                      "base_buckets": st_build["base_buckets"],
                      "overflow_buckets": st_build["overflow_buckets"],
                      "max_chain": st_build["max_chain"],
                      "realised_load_factor": st_build["load_factor"],
                      "utilization": st_build["utilization"],
                      "table_MB": st_build["pool_bytes"] / 2**20,
                      "digest_after_ops": digest(g)}
                res.append(pt)
                print(json.dumps(pt), flush=True)
                g.close()
    digests = {p["digest_after_ops"] for p in res}
    summary = {"points": len(res), "geometry_invariant": len(digests) == 1,
               "graph": f"grid {rows_}x{cols}, |E|={bs.size}"}
    print(json.dumps(summary))
    if out:
        json.dump({"summary": summary, "points": res}, open(out, "w"), indent=1)


if __name__ == "__main__":
    main()
