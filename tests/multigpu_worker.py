"""torchrun worker: P ranks, one GPU each, graph sharded by source vertex (owner
u mod P).  Every rank feeds its own slice of each batch; rank 0 gathers the shard
exports and compares the union with the unsharded oracle."""
import os
import sys

import numpy as np
import torch
import torch.distributed as dist

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import workloads as wl  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph, get_unique_id  # noqa: E402


def main():
    rank, P = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    local = int(os.environ["LOCAL_RANK"])
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist.init_process_group("nccl", device_id=dev)
    obj = [get_unique_id() if rank == 0 else None]
    dist.broadcast_object_list(obj, src=0)
    nv = 50_000
    g = Graph(nv, rank=rank, nranks=P, nccl_unique_id=obj[0])
    cu = lambda a: torch.from_numpy(np.ascontiguousarray(a, np.uint32)).to(dev)  # noqa: E731
    batches = []
    for b in range(3):
        n = 100_000
        off = n * rank // P
        cnt = n * (rank + 1) // P - off
        s, d, w = wl.uniform_edges(31, b, cnt, nv, offset=off)
        added = g.insert_edges(cu(s), cu(d), cu(w), count=True)
        batches.append(("ins", b, added))
    qs, qd, _ = wl.uniform_edges(31, 1, 40_000, nv, offset=rank * 40_000)
    f, qw = g.query_edges(cu(qs), cu(qd))
    ds, dd, _ = wl.uniform_edges(31, 2, 30_000, nv, offset=rank * 30_000)
    removed = g.delete_edges(cu(ds), cu(dd), count=True)
    ids = wl.uniform_u32(31, 9, 50, nv, offset=rank * 50)
    g.delete_vertices(cu(ids))
    ro, dst, wt = g.export(device=False)
    shard = (ro, dst, wt)
    out = [None] * P if rank == 0 else None
    dist.gather_object((shard, qs, qd, f.cpu().numpy(), qw.cpu().numpy(), ds, dd, ids,
                        [x[2] for x in batches], removed), out, dst=0)
    if rank == 0:
        from oracle import Oracle
        from oracle.compare import Candidates, compare_export, compare_queries
        o = Oracle(nv)
        for b in range(3):
            s, d, w = wl.uniform_edges(31, b, 100_000, nv)
            st, added = o.insert_edges(s, d, w)
            assert added == out[0][8][b], (added, out[0][8][b])
        cand = Candidates(*o.candidates())
        for k in range(P):
            st, rf, rw = o.query_edges(out[k][1], out[k][2])
            errs = compare_queries(out[k][1], out[k][2], out[k][3], out[k][4], rf, rw, cand)
            assert not errs, errs
        allds = np.concatenate([out[k][5] for k in range(P)])
        alldd = np.concatenate([out[k][6] for k in range(P)])
        assert o.delete_edges(allds, alldd)[1] == out[0][9]
        o.delete_vertices(np.concatenate([out[k][7] for k in range(P)]))
        # merge shard exports: local row r of rank k is global vertex r*P + k
        ro_g, d_g, w_g = o.export()
        deg = np.diff(ro_g).astype(np.int64)
        cu_, cv_, cw_ = o.candidates()
        for k in range(P):
            m = (cu_ % P) == k
            cand_k = Candidates(cu_[m] // P, cv_[m], cw_[m])
            ro, dst, wt = out[k][0]
            rows = np.arange(ro.size - 1) * P + k
            want_ro = np.concatenate([[0], np.cumsum(deg[rows])]).astype(np.uint64)
            sel = np.concatenate([np.arange(ro_g[u], ro_g[u + 1]) for u in rows]).astype(np.int64)
            errs = compare_export((ro, dst, wt), (want_ro, d_g[sel], w_g[sel]), cand_k)
            assert not errs, (k, errs)
        print("MULTIGPU OK", flush=True)
    g.close()
    dist.barrier()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
