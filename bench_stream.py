"""bench.py configs 4 and 5.

cfg4 — mixed stream on R-MAT scale 24 (Graph500 a,b,c = .57,.19,.19, edge factor 16,
permuted IDs, seed 4): bulk build, then per step: insert 2^22 new R-MAT edges, query
2^22 (half sampled from the base edges, half uniform), delete 2^21 (half base edges,
half uniform), delete 2^12 vertices (1/4 drawn from the top-1% out-degree vertices)
and insert 2^16 edges leaving the just-deleted IDs (vertex re-insertion).
Sharded by source vertex at N > 1, each rank feeding 1/N of every batch.

cfg5 — dynamic triangle counting (§VI-C2): R-MAT scale 22 symmetrised
(undirected mode), then per step: insert 2^22 new R-MAT edges (both directions) and
count triangles by hash intersection.  At N > 1 every GPU holds a replica, inserts
the whole batch, and counts the wedges of u mod N == rank (one all-reduce).
"""
from __future__ import annotations

import json
import os
import time

import numpy as np

import workloads as wl
from bench import (L2_NOTE, METRIC, UNIT, ClockSampler, L2Flush, config_block, dist_env,
                   load_peaks, make_coll, model_bytes, parallelism_label, slice_of)


def _setup(args):
    import torch
    world, rank, local = dist_env()
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    return torch, world, rank, local, dev, make_coll(world, rank, dev)


def _clock(local):
    vis = os.environ.get("CUDA_VISIBLE_DEVICES")
    return ClockSampler(vis.split(",")[local] if vis else local)


def _max(torch, pg, dev, vals):
    t = torch.tensor(vals, dtype=torch.float64, device=dev)
    if pg:
        pg.all_reduce(t, "max")
    return t.tolist()


def _sum(torch, pg, dev, vals):
    t = torch.tensor(vals, dtype=torch.float64, device=dev)
    if pg:
        pg.all_reduce(t, "sum")
    return t.tolist()


# ------------------------------------------------------------------ cfg4 ----
def run_mixed(args, cfg):
    torch, world, rank, local, dev, pg = _setup(args)
    from paper_conf_ipps_awadapo20_b200 import Graph
    gkw = pg.graph_kwargs() if pg else {}
    nv, m, seed, scale, abc = cfg["nv"], cfg["m"], cfg["seed"], cfg["scale"], cfg["abc"]
    S = args.bucket_bytes
    t0 = time.perf_counter()
    off, cnt = slice_of(m, rank, world)
    bs, bd = wl.rmat_edges(seed, 0, cnt, scale, abc, offset=off)
    bw = wl.weights(seed, 0, cnt, offset=off)
    deg = torch.bincount(torch.from_numpy(bs.astype(np.int64)).to(dev), minlength=nv)
    if pg:
        pg.all_reduce(deg, "sum")
    hints = deg.to(torch.int32).contiguous()
    top = torch.topk(deg, nv // 100).indices.to(torch.int64).cpu().numpy().astype(np.uint32)
    gen_s = time.perf_counter() - t0
    cu = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)  # noqa: E731
    ev = lambda: torch.cuda.Event(enable_timing=True)  # noqa: E731
    torch.cuda.synchronize()
    if pg:
        pg.barrier()
    a0, a1 = ev(), ev()
    g = Graph(nv, hints, bucket_bytes=S, load_factor=args.load_factor, rank=rank, nranks=world,
              set_variant=args.variant == "set", **gkw)
    BS, BD, BW = cu(bs), cu(bd), cu(bw)
    torch.cuda.synchronize()
    a0.record()
    added0 = g.insert_edges(BS, BD, BW, count=True)
    a1.record()
    torch.cuda.synchronize()
    bulk_ms = _max(torch, pg, dev, [a0.elapsed_time(a1)])[0]
    del BS, BD, BW
    flush = L2Flush(dev)
    IB, QB, DB, VB, RB = 1 << 22, 1 << 22, 1 << 21, 1 << 12, 1 << 16
    names = ["insert", "query", "delete", "delete_vertices", "reinsert"]
    tot = dict.fromkeys(names, 0.0)
    nops = dict.fromkeys(names, 0)
    clock = None
    for step in range(args.warmup + args.steps):
        timed = step >= args.warmup
        st = 1 + step
        io, ic = slice_of(IB, rank, world)
        s1, d1 = wl.rmat_edges(seed, st, ic, scale, abc, offset=io)
        w1 = wl.weights(seed, st, ic, offset=io)
        qo, qc = slice_of(QB, rank, world)
        half = qc // 2
        ls, ld = wl.rmat_edges(seed, 0, 0, scale, abc,
                               index=wl.uniform_index(seed, 5000 + st * 64 + rank, half, m))
        us, ud, _ = wl.uniform_edges(seed, 6000 + st, qc - half, nv, weights=False, offset=qo)
        qs, qd = np.concatenate([ls, us]), np.concatenate([ld, ud])
        do, dc = slice_of(DB, rank, world)
        half = dc // 2
        xs, xd = wl.rmat_edges(seed, 0, 0, scale, abc,
                               index=wl.uniform_index(seed, 7000 + st * 64 + rank, half, m))
        ys, yd, _ = wl.uniform_edges(seed, 8000 + st, dc - half, nv, weights=False, offset=do)
        ds, dd = np.concatenate([xs, ys]), np.concatenate([xd, yd])
        vo, vc = slice_of(VB, rank, world)
        nh = vc // 4
        hub = top[wl.uniform_u32(seed, 9000 + st, nh, top.size, offset=vo)]
        ids = np.concatenate([hub, wl.uniform_u32(seed, 9100 + st, vc - nh, nv, offset=vo)])
        ro_, rc = slice_of(RB, rank, world)
        rs = ids[wl.uniform_u32(seed, 9200 + st, rc, ids.size, offset=ro_)] if ids.size else \
            np.zeros(rc, np.uint32)
        rd, _, rw = wl.uniform_edges(seed, 9300 + st, rc, nv, offset=ro_)
        dev_in = [(cu(s1), cu(d1), cu(w1)), (cu(qs), cu(qd)), (cu(ds), cu(dd)), (cu(ids),),
                  (cu(rs), cu(rd), cu(rw))]
        if timed and step == args.warmup:
            torch.cuda.synchronize()
            if pg:
                pg.barrier()
            g.profile_enable(True)
            clock = _clock(local)
        calls = [lambda x: g.insert_edges(*x), lambda x: g.query_edges(*x),
                 lambda x: g.delete_edges(*x), lambda x: g.delete_vertices(*x),
                 lambda x: g.insert_edges(*x)]
        sizes = [ic, qc, dc, vc, rc]
        for k, (name, fn, inp) in enumerate(zip(names, calls, dev_in)):
            torch.cuda.synchronize()
            if pg:
                pg.barrier()
            flush()
            e0, e1 = ev(), ev()
            e0.record()
            fn(inp)
            e1.record()
            torch.cuda.synchronize()
            if timed:
                tot[name] += e0.elapsed_time(e1)
                nops[name] += sizes[k]
    prof = g.profile_read()
    clocks = clock.stop() if clock else None
    g.profile_enable(False)
    times = _max(torch, pg, dev, [tot[n] for n in names])
    counts = _sum(torch, pg, dev, [nops[n] for n in names])
    tms = dict(zip(names, times))
    cnt_ = dict(zip(names, counts))
    edge_ops = cnt_["insert"] + cnt_["query"] + cnt_["delete"] + cnt_["reinsert"]
    total_ms = sum(times)
    value = edge_ops / (total_ms * 1e3)
    K = args.steps
    ops = {n: {"ms_per_step": tms[n] / K,
               ("M_vertices_s" if n == "delete_vertices" else "M_edges_s"):
                   cnt_[n] / (tms[n] * 1e3) if tms[n] else None} for n in names}
    peak, peak_src = load_peaks()
    # dominant kernel: the streaming purge sweep reads every allocated bucket once
    st_ = g.stats()
    sweep_bytes = st_["bump_bytes"]
    vms = prof["kernel_ms"]["vertex_purge"]
    vl = max(1, prof["kernel_launches"]["vertex_purge"])
    kms = prof["kernel_ms"]
    dom = max(kms, key=lambda k: kms[k])
    roofline = {"bound": "hbm", "kernel": dom, "unit": "GB/s", "peak": peak,
                "peak_source": peak_src, "traffic": None,
                "kernel_share_of_step": kms[dom] / total_ms if total_ms else None}
    if dom == "vertex_purge":
        roofline["achieved"] = sweep_bytes * vl / (vms * 1e-3) / 1e9
        roofline["algorithmic_bytes_per_launch"] = sweep_bytes
        roofline["note"] = "purge sweep + clear: model bytes = allocated buckets x bucket bytes"
    else:
        mb = model_bytes(S or st_["table_bytes"] / max(1, st_["base_buckets"] + st_["overflow_buckets"]))
        per = {"insert": mb["insert_new"], "query": mb["query"], "delete": mb["delete_hit"]}
        nb = cnt_[dom] / world * per.get(dom, mb["query"])
        roofline["achieved"] = nb / (kms[dom] * 1e-3) / 1e9
        roofline["algorithmic_bytes_per_launch"] = nb / max(1, prof["kernel_launches"][dom])
    roofline["frac"] = roofline["achieved"] / peak
    line = {
        "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": K,
        "warmup": args.warmup, "ms_per_step": total_ms / K, "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "u32",
        "data": "synthetic (seeded counter-based generators, workloads/gen.c)",
        "config": {"workload": f"cfg4: {cfg['name']} |V|={nv:,} |E|={m:,} generated; step = "
                               f"insert {IB:,} + query {QB:,} + delete {DB:,} edges + delete "
                               f"{VB:,} vertices + re-insert {RB:,} edges (global)",
                   "bucket_bytes": S, "load_factor": args.load_factor,
                   "l2": L2_NOTE,
                   "parallelism": parallelism_label(world)},
        "ops": ops, "bulk_build": {"insert_ms": bulk_ms, "unique_added": int(added0)},
        "roofline": roofline, "gpu_launches": prof["launches"], "clocks": clocks,
        "graph": {k: st_[k] for k in ("live_pairs", "tombstones", "max_chain", "pool_bytes")},
        "gen_s": gen_s, "cpu_baseline": None, "e2e": None,
    }
    if rank == 0:
        print(json.dumps(line), flush=True)
    g.close()
    if pg:
        pg.close()
    return 0


# ------------------------------------------------------------------ cfg5 ----
def run_tc(args, cfg):
    torch, world, rank, local, dev, pg = _setup(args)
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv, m, seed, scale, abc = cfg["nv"], cfg["m"], cfg["seed"], cfg["scale"], cfg["abc"]
    S = args.bucket_bytes
    t0 = time.perf_counter()
    bs, bd = wl.rmat_edges(seed, 0, m, scale, abc)  # every GPU holds a replica
    deg = torch.bincount(torch.from_numpy(np.concatenate([bs, bd]).astype(np.int64)).to(dev),
                         minlength=nv)
    hints = deg.to(torch.int32).contiguous()
    gen_s = time.perf_counter() - t0
    cu = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)  # noqa: E731
    ev = lambda: torch.cuda.Event(enable_timing=True)  # noqa: E731
    # the paper counts triangles on the set variant (keys only)
    variant = args.variant or "set"
    g = Graph(nv, hints, bucket_bytes=S, load_factor=args.load_factor, directed=False,
              set_variant=variant == "set")
    a0, a1 = ev(), ev()
    BS, BD = cu(bs), cu(bd)
    torch.cuda.synchronize()
    a0.record()
    g.insert_edges(BS, BD)
    a1.record()
    torch.cuda.synchronize()
    bulk_ms = a0.elapsed_time(a1)
    del BS, BD
    flush = L2Flush(dev)
    IB = 1 << 22
    t_ins = t_tc = 0.0
    wedges = []  # edgeExist probes of each timed TC, counted on the graph it ran on
    tc_steps = []  # device ms of each timed TC (this rank)
    tri = []
    clock = None
    # warm-up steps count triangles on the bulk-built graph only; the timed steps are
    # the paper's dynamic iterations (insert 2^22, then TC)
    for step in range(args.warmup + args.steps):
        timed = step >= args.warmup
        s1, d1 = wl.rmat_edges(seed, 1 + max(0, step - args.warmup), IB if timed else 0, scale, abc)
        S1, D1 = cu(s1), cu(d1)
        if timed and step == args.warmup:
            torch.cuda.synchronize()
            if pg:
                pg.barrier()
            g.profile_enable(True)
            clock = _clock(local)
        torch.cuda.synchronize()
        if pg:
            pg.barrier()
        flush()
        e0, e1, e2 = ev(), ev(), ev()
        e0.record()
        g.insert_edges(S1, D1)
        e1.record()
        c = g.triangle_count(rank, world)
        e2.record()
        torch.cuda.synchronize()
        if timed:
            t_ins += e0.elapsed_time(e1)
            t_tc += e1.elapsed_time(e2)
            tc_steps.append(e1.elapsed_time(e2))
            tri.append(c)
            # the graph grows every step: count this TC's probes now (untimed, host)
            wedges.append(_wedges(g, rank, world))
    prof = g.profile_read()
    clocks = clock.stop() if clock else None
    g.profile_enable(False)
    # wedges probed = sum over u of C(|N+(u)|, 2) (the oriented out-degrees)
    st_ = g.stats()
    t_ins, t_tc = _max(torch, pg, dev, [t_ins, t_tc])
    tri = [int(x) for x in _sum(torch, pg, dev, tri)]
    K = args.steps
    wk = prof["kernel_ms"]["tc"]
    nl = max(1, prof["kernel_launches"]["tc"])
    wedges = [int(x) for x in _sum(torch, pg, dev, wedges)]  # all parts, per step
    wedge_ops = sum(wedges) / K  # mean per TC
    edge_ops = 2 * IB * K + sum(wedges)
    total_ms = t_ins + t_tc
    value = edge_ops / (total_ms * 1e3)
    peak, peak_src = load_peaks()
    # one bucket of A_v + the streamed candidate id; adaptive layout: the
    # mean bytes of a linked bucket
    Sb = S or st_["table_bytes"] / max(1, st_["base_buckets"] + st_["overflow_buckets"])
    bytes_per_probe = Sb + 4
    # wk covers the nl timed launches (one per step); their probes are sum(wedges)
    roofline = {"bound": "hbm", "kernel": (f"k_tc_wedges_flat<{S // 16},{variant}>" if S else "k_tc_wedges<adaptive,{variant}>"),
                "unit": "GB/s",
                "achieved": sum(wedges) / world * bytes_per_probe / (wk * 1e-3) / 1e9,
                "peak": peak, "peak_source": peak_src, "traffic": None,
                "algorithmic_bytes_per_launch": sum(wedges) / world * bytes_per_probe / nl,
                "note": "model bytes = one bucket of A_v + 4 B per wedge probe, wedges counted "
                        "per step on the graph each TC ran on; probes largely hit L2 (small "
                        "tables reused), so the model may exceed the HBM copy peak — the DRAM "
                        "fraction from ncu is `dram_frac`",
                "kernel_share_of_step": wk / total_ms if total_ms else None}
    roofline["frac"] = roofline["achieved"] / peak
    tpath = os.path.join(os.path.dirname(os.path.abspath(__file__)), "profiles", "ncu_traffic.json")
    try:
        ent = json.load(open(tpath)).get(f"cfg5/tc/s{S}")
    except (OSError, ValueError):
        ent = None
    if ent:  # ncu DRAM bytes of one wedge launch over its ncu duration
        roofline["traffic"] = ent["dram_bytes_per_launch"]
        roofline["dram_frac"] = ent["dram_bytes_per_launch"] / (ent["ncu_duration_ms"] * 1e-3) / 1e9 / peak
        roofline["dram_source"] = ent.get("source")
    line = {
        "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": K,
        "warmup": args.warmup, "ms_per_step": total_ms / K, "higher_is_better": True,
        "scaling": "strong" if world > 1 else "weak", "vs_baseline": None, "dtype": "u32",
        "data": "synthetic (seeded counter-based generators, workloads/gen.c)",
        "config": {"workload": f"cfg5: {cfg['name']} |V|={nv:,}, {m:,} generated edges "
                               f"symmetrised; step = insert {IB:,} new undirected edges + TC "
                               f"(edge ops counted: 2 directed inserts per edge + 1 edgeExist "
                               f"per wedge)",
                   "bucket_bytes": S, "load_factor": args.load_factor, "variant": variant,
                   "l2": L2_NOTE + " (before every step)",
                   "parallelism": parallelism_label(world, f"replicas, wedges split by u mod {world},")},
        "tc": {"triangles_per_step": tri, "tc_ms_per_step": t_tc / K,
               "tc_ms_steps": [round(x, 3) for x in tc_steps],
               "insert_ms_per_step": t_ins / K, "wedges_per_tc": wedges,
               "wedge_G_per_s": sum(wedges) / (t_tc * 1e-3) / 1e9,
               "insert_M_edges_s": 2 * IB / (t_ins / K * 1e3)},
        "bulk_build": {"insert_ms": bulk_ms},
        "roofline": roofline, "gpu_launches": prof["launches"], "clocks": clocks,
        "graph": {k: st_[k] for k in ("live_pairs", "max_chain", "pool_bytes")},
        "gen_s": gen_s, "cpu_baseline": None, "e2e": None,
    }
    if rank == 0:
        print(json.dumps(line), flush=True)
    g.close()
    if pg:
        pg.close()
    return 0


def _wedges(g, part, nparts):
    """sum over u with u % nparts == part of C(d+(u), 2), d+ = oriented out-degree by
    rank (degree, id) — the number of edgeExist probes one TC issues (accounting)."""
    ro, dst, _ = g.export_numpy()
    deg = np.diff(ro.astype(np.int64))
    rows = np.repeat(np.arange(deg.size, dtype=np.int64), deg)
    d = dst.astype(np.int64)
    keep = (deg[d] > deg[rows]) | ((deg[d] == deg[rows]) & (d > rows))
    keep &= (rows % nparts) == part
    dp = np.bincount(rows[keep], minlength=deg.size).astype(np.int64)
    return int((dp * (dp - 1) // 2).sum())
