#!/usr/bin/env python3
"""Benchmark: batched edge insert / query / delete rate (M edges/s) on B200.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
                    [--config cfg2|cfg3] [--batch-log2 24] [--bucket-bytes 128]

Workload (BASELINE.json configs[1]): LJ-like R-MAT, |V| = 4,847,571,
|E| = 68,993,773 (scale 23, (a,b,c) = (.50,.20,.20), permuted IDs, seed 2), bulk-built
with exact degree hints.  One STEP = one pass of the hot path over one
batch: insert B uniform random edges between existing vertices, query B
edges (half sampled from the graph, half uniform), delete B edges (half of the
inserted ones, half uniform pairs: mostly misses).  After the timed step
the other half of the inserted edges is deleted untimed, so every step starts from
the bulk-built graph.  `value` = 3*B*K / (device time of the K steps), inputs
resident in HBM, L2 flushed (256 MiB write, then a 256 MiB read) before every op.  `e2e` repeats the steps through the same API with
pinned HOST buffers (H2D of inputs and D2H of query answers inside the timed region).

At N > 1 (torchrun, one process per GPU) every rank holds the rows it owns
(owner(u) = u mod N) and contributes its own B-edge slice of every batch (weak
scaling); the library routes each op to its owner over NCCL.

`--impl reference` times the CPU oracle (oracle/, one std::unordered_map per vertex)
on a bounded row sample of the same workload (1/64 of the rows, hashed), run by T
host threads that own disjoint rows.
"""
from __future__ import annotations

import argparse
import csv
import io
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)
if __name__ == "__main__":  # bench_stream imports `bench`: the same module, not a copy
    sys.modules.setdefault("bench", sys.modules[__name__])

import workloads as wl  # noqa: E402

METRIC = "batched edge insert/delete/query rate (M edges/s) at 1/2/4/8 B200"
UNIT = "M edges/s"

CONFIGS = {
    "cfg2": dict(name="LJ-like R-MAT", nv=4_847_571, m=68_993_773, scale=23, abc=wl.LJLIKE,
                 seed=2, kind="rmat"),
    "cfg3": dict(name="road-like grid", rows=4894, cols=4894, p=0.6025, seed=3, kind="grid"),
    "cfg4": dict(name="R-MAT scale 24 mixed stream", nv=1 << 24, m=1 << 28, scale=24,
                 abc=wl.GRAPH500, seed=4, kind="rmat", stream=True),
    "cfg5": dict(name="R-MAT scale 22 symmetrised, dynamic TC", nv=1 << 22, m=1 << 26, scale=22,
                 abc=wl.GRAPH500, seed=5, kind="rmat", tc=True),
}
SAMPLE_MOD = 64  # oracle row sample: 1/64 of the rows, by a multiplicative hash of u


def in_sample(u):
    """rows of the oracle sample: the top 6 bits of u * 0x9E3779B97F4A7C15 (mod 2^64)
    are 0 — 1/64 of the rows, spread over every residue mod T (a plain u % 64 == 0
    sample would put every sampled row on one oracle thread)."""
    h = np.asarray(u, np.uint64) * np.uint64(0x9E3779B97F4A7C15)
    return (h >> np.uint64(58)) == 0


# ----------------------------------------------------------------- helpers --
_RANK = threading.local()  # --inproc: (world, rank, local) of this rank thread


def dist_env():
    if getattr(_RANK, "env", None):
        return _RANK.env
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


class DistColl:
    """The bench's own collectives over torch.distributed (one process per GPU, the
    layout the driver launches); the library's rank communicator is NCCL."""

    def __init__(self, dev, rank):
        import torch.distributed as dist
        from paper_conf_ipps_awadapo20_b200 import get_unique_id
        dist.init_process_group("nccl", device_id=dev)
        self.dist = dist
        obj = [get_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        self.uid = obj[0]

    def graph_kwargs(self):
        return {"nccl_unique_id": self.uid}

    def barrier(self):
        self.dist.barrier()

    def all_reduce(self, t, op="sum"):
        self.dist.all_reduce(t, op=self.dist.ReduceOp.MAX if op == "max" else self.dist.ReduceOp.SUM)

    def close(self):
        self.dist.barrier()
        self.dist.destroy_process_group()


class ThreadColl:
    """Dry run of the N > 1 path without N GPUs (`--inproc N`): the ranks are threads
    of this process over an in-process rank group (`RankGroup`), spread round-robin
    over the visible GPUs; the bench's collectives meet at a thread barrier.  It
    exercises the sharded bench and library code paths (slices, routing, answers,
    max-over-ranks timing); its rates are not a scaling measurement."""

    def __init__(self, shared, rank):
        self.s, self.rank = shared, rank

    def graph_kwargs(self):
        return {"group": self.s["group"]}

    def barrier(self):
        self.s["barrier"].wait()

    def all_reduce(self, t, op="sum"):
        import torch
        slots = self.s["slots"]
        slots[self.rank] = t.detach().cpu().clone()
        self.barrier()
        acc = slots[0].clone()
        for x in slots[1:]:
            acc = torch.maximum(acc, x) if op == "max" else acc + x
        self.barrier()
        t.copy_(acc.to(t.device))

    def close(self):
        self.barrier()


def parallelism_label(world, what="source-vertex sharding"):
    lab = f"{what} x{world}" if world > 1 else "single GPU"
    if getattr(_RANK, "shared", None):
        lab += " (in-process rank group dry run: --inproc)"
    return lab


def make_coll(world, rank, dev):
    if world == 1:
        return None
    shared = getattr(_RANK, "shared", None)
    return ThreadColl(shared, rank) if shared else DistColl(dev, rank)


def run_inproc(args, fn):
    """--inproc N: N rank threads, each with its own stream (dry run, see ThreadColl)."""
    import torch
    from paper_conf_ipps_awadapo20_b200 import RankGroup
    n = args.inproc
    ndev = max(1, torch.cuda.device_count())
    shared = {"group": RankGroup(n), "barrier": threading.Barrier(n), "slots": [None] * n}
    errors = []

    def rank_main(r):
        try:
            _RANK.env = (n, r, r % ndev)
            _RANK.shared = shared
            torch.cuda.set_device(r % ndev)
            with torch.cuda.stream(torch.cuda.Stream()):
                fn(args, CONFIGS[args.config])
        except BaseException as e:  # noqa: BLE001
            errors.append((r, repr(e)))
            shared["barrier"].abort()

    th = [threading.Thread(target=rank_main, args=(r,)) for r in range(n)]
    for t in th:
        t.start()
    for t in th:
        t.join()
    if errors:
        print(json.dumps({"inproc_errors": errors}), file=sys.stderr)
        return 1
    return 0


def slice_of(n, rank, world):
    a = n * rank // world
    b = n * (rank + 1) // world
    return a, b - a


L2_NOTE = ("flushed before every timed op: 256 MiB written, then another 256 MiB read, so the "
           "flush's own dirty lines are written back before the timed region and the op starts "
           "from a clean, cold L2; tables >> L2")


class L2Flush:
    """L2 flush between timed ops: write a buffer larger than L2 (evicts our data), then
    read a second one (writes the first one's dirty lines back now, not inside the next
    timed op: a 2^16-op insert measured 36.7 us behind the write-only flush, 25.7 us
    back to back; the read leaves L2 clean and cold)."""

    def __init__(self, dev):
        import torch
        self.w = torch.empty(256 << 20, dtype=torch.uint8, device=dev)
        self.r = torch.zeros(32 << 20, dtype=torch.int64, device=dev)  # 256 MiB

    def __call__(self):
        self.w.zero_()
        self.r.sum()


def load_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


def build_base(cfg, rank=0, world=1):
    """This rank's slice of the base edge list + global degree hints (numpy)."""
    if cfg["kind"] == "rmat":
        nv, m = cfg["nv"], cfg["m"]
        off, cnt = slice_of(m, rank, world)
        s, d = wl.rmat_edges(cfg["seed"], 0, cnt, cfg["scale"], cfg["abc"], nv=nv, offset=off)
        w = wl.weights(cfg["seed"], 0, cnt, offset=off)
    else:
        nv = cfg["rows"] * cfg["cols"]
        s_all, d_all = wl.grid_edges(cfg["seed"], cfg["rows"], cfg["cols"], cfg["p"])
        m = s_all.size
        off, cnt = slice_of(m, rank, world)
        s, d = s_all[off:off + cnt].copy(), d_all[off:off + cnt].copy()
        w = wl.weights(cfg["seed"], 0, cnt, offset=off)
    return nv, m, s, d, w


def live_sample(cfg, base, n, seed_stream, rank, world):
    """n edges sampled uniformly from the base edge list (regenerated by id, so any
    rank can produce any edge)."""
    m = cfg["m"] if cfg["kind"] == "rmat" else base[1]
    idx = wl.uniform_index(cfg["seed"], seed_stream, n, m)
    if cfg["kind"] == "rmat":
        return wl.rmat_edges(cfg["seed"], 0, 0, cfg["scale"], cfg["abc"], nv=cfg["nv"], index=idx)
    s_all, d_all = base[2]
    return s_all[idx], d_all[idx]


def step_batch(cfg, nv, B, step, rank, world, base):
    """Insert batch (uniform over existing vertices), query batch (half live: sampled
    from the base graph, half uniform) and delete batch (half live: the first half of
    this step's insert batch, half uniform pairs — mostly misses, as random deletes
    are in the paper)."""
    seed = cfg["seed"]
    s, d, w = wl.uniform_edges(seed, 1000 + step, B, nv, offset=rank * B)
    half = B // 2
    ls, ld = live_sample(cfg, base, half, 5000 + step * world + rank, rank, world)
    us, ud, _ = wl.uniform_edges(seed, 7000 + step, B - half, nv, weights=False,
                                 offset=rank * (B - half))
    qs = np.concatenate([ls, us])
    qd = np.concatenate([ld, ud])
    ys, yd, _ = wl.uniform_edges(seed, 8000 + step, B - half, nv, weights=False,
                                 offset=rank * (B - half))
    xs = np.concatenate([s[:half], ys])
    xd = np.concatenate([d[:half], yd])
    return (s, d, w), (qs, qd), (xs, xd)


def model_bytes(S):
    """Algorithmic bytes per op outcome: input + 32-B
    directory sector + one S-byte bucket + 32-B pair/tombstone write + 32-B degree
    write-back; query adds the 5-B answer."""
    return {
        "insert_new": 12 + 32 + S + 32 + 32,
        "insert_replace": 12 + 32 + S + 32,
        "delete_hit": 8 + 32 + S + 32 + 32,
        "delete_miss": 8 + 32 + S,
        "query": 8 + 32 + S + 5,
        "selfloop_insert": 12,
        "selfloop_other": 8,
    }


class ClockSampler:
    """nvidia-smi clocks / throttle reasons sampled every 200 ms during the timed region."""

    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu_index):
        self.proc = None
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--id={gpu_index}", f"--query-gpu={self.FIELDS}",
                 "--format=csv,noheader,nounits", "-lms", "200"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except (OSError, ValueError):
            self.proc = None

    def stop(self):
        if self.proc is None:
            return None
        self.proc.terminate()
        try:
            out, _ = self.proc.communicate(timeout=5)
        except subprocess.TimeoutExpired:
            self.proc.kill()
            out, _ = self.proc.communicate()
        rows = [r for r in csv.reader(io.StringIO(out)) if len(r) >= 9]
        if not rows:
            return None
        sm = [float(r[1]) for r in rows if r[1].strip().replace(".", "").isdigit()]
        mx = [float(r[2]) for r in rows if r[2].strip().replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i in range(4)
                          if r[5 + i].strip().lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None,
                "sm_max_mhz": max(mx) if mx else None, "reasons": reasons,
                "samples": len(rows)}


def host_cpu():
    """(model name, logical CPUs usable by this process) of the host."""
    model = "unknown"
    try:
        for ln in open("/proc/cpuinfo"):
            if ln.startswith("model name"):
                model = ln.split(":", 1)[1].strip()
                break
    except OSError:
        pass
    try:
        n = len(os.sched_getaffinity(0))
    except AttributeError:
        n = os.cpu_count() or 1
    return model, n


class ThreadedOracle:
    """The oracle as it stands on T host threads (thread t applies the
    ops of the vertices u with u % T == t, in batch order), over the row sample
    in_sample() (1/64 of the rows) of the workload.  T = the host's usable CPUs (at
    most 64)."""

    def __init__(self, nv, base_s, base_d, base_w):
        from oracle import Oracle
        model, ncpu = host_cpu()
        self.T = max(1, min(ncpu, 64))
        self.model, self.ncpu = model, ncpu
        self.o = Oracle(nv, threads=self.T)
        m = in_sample(base_s)
        self.sample_edges = int(m.sum())
        self.o.insert_edges(base_s[m], base_d[m], base_w[m])

    @staticmethod
    def sample(s, *rest):
        """the sampled rows' ops (input preparation, untimed)"""
        m = in_sample(s)
        return (s[m],) + tuple(r[m] for r in rest)

    def step(self, s, d, w, qs, qd, xs, xd):
        """one step (insert, query, delete) restricted to the sample; -> (ops, seconds)"""
        a, b, c = self.sample(s, d, w)
        x, y = self.sample(qs, qd)
        p, q = self.sample(xs, xd)
        t0 = time.perf_counter()
        self.o.insert_edges(a, b, c)
        self.o.query_edges(x, y)
        self.o.delete_edges(p, q)
        return a.size + x.size + p.size, time.perf_counter() - t0

    def delete(self, s, d):
        self.o.delete_edges(*self.sample(s, d))

    def describe(self):
        return f"{self.T} threads of {self.ncpu} usable CPUs ({self.model})"


def cpu_baseline(cfg, nv, base_s, base_d, base_w, batches, budget_s=12.0):
    """The oracle (as it stands, T threads partitioned by row) on the row sample
    u % 64 == 0 of the same workload: build the sampled rows (untimed), then time the
    step ops restricted to those rows until ~budget_s of wall time."""
    to = ThreadedOracle(nv, base_s, base_d, base_w)
    ops = 0
    t = 0.0
    steps = 0
    while t < budget_s and steps < 64:
        (s, d, w), (qs, qd), (xs, xd) = batches[steps % len(batches)]
        k, dt = to.step(s, d, w, qs, qd, xs, xd)
        to.delete(s[len(s) // 2:], d[len(d) // 2:])  # untimed, as in the GPU steps
        ops += k
        t += dt
        steps += 1
    return {"value": ops / t / 1e6, "unit": UNIT, "cores": to.T, "kind": "oracle",
            "host": to.describe(),
            "sample": f"1/{SAMPLE_MOD} of the rows (hashed) of {cfg['name']} ({to.sample_edges} of "
                      f"{base_s.size} base edges); {steps} steps of insert+query+delete "
                      f"restricted to those rows ({ops} ops, {t:.1f} s wall on {to.T} threads)"}


# --------------------------------------------------------------- reference --
def run_reference(args, cfg):
    world, rank, _ = dist_env()
    if rank != 0:
        return 0
    nv, m_total, base_s, base_d, base_w = build_base(cfg)
    B = 1 << args.batch_log2
    to = ThreadedOracle(nv, base_s, base_d, base_w)
    times, ops = [], []
    for step in range(args.warmup + args.steps):
        (s, d, w), (qs, qd), (xs, xd) = step_batch(cfg, nv, B, step, 0, 1,
                                                   (None, m_total, (base_s, base_d)))
        k, dt = to.step(s, d, w, qs, qd, xs, xd)
        to.delete(s[B // 2:], d[B // 2:])  # as in our arm: untimed
        if step >= args.warmup:
            times.append(dt)
            ops.append(k)
    value = sum(ops) / sum(times) / 1e6
    sample = (f"1/{SAMPLE_MOD} of the rows (hashed) of {cfg['name']}; each step = the step's insert/query/"
              f"delete batches restricted to those rows (~{int(np.mean(ops))} ops); "
              f"{to.describe()}")
    line = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world,
        "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": 1e3 * sum(times) / len(times), "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "u32", "data": "synthetic",
        "config": config_block(cfg, args, nv, m_total, B, world),
        "cpu_baseline": {"value": value, "unit": UNIT, "cores": to.T, "kind": "oracle",
                         "sample": sample},
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


def config_block(cfg, args, nv, m, B, world):
    if cfg["kind"] == "rmat":
        wname = (f"{args.config}: {cfg['name']} |V|={nv:,} |E|={m:,} (scale {cfg['scale']}, "
                 f"abc={cfg['abc']}), bulk-built with degree hints; step = insert {B:,} + "
                 f"query {B:,} + delete {B:,} edges per GPU")
    else:
        wname = (f"{args.config}: {cfg['name']} {cfg['rows']}x{cfg['cols']} |V|={nv:,} "
                 f"|E|={m:,}; step = insert {B:,} + query {B:,} + delete {B:,} edges per GPU")
    return {"workload": wname, "batch_per_gpu": B, "global_batch": B * world,
            "bucket_bytes": args.bucket_bytes, "load_factor": args.load_factor,
            "variant": args.variant or "map",
            "l2": L2_NOTE,
            "parallelism": parallelism_label(world)}


# -------------------------------------------------------------------- ours --
def run_ours(args, cfg):
    import torch
    world, rank, local = dist_env()
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    from paper_conf_ipps_awadapo20_b200 import Graph
    pg = make_coll(world, rank, dev)
    gkw = pg.graph_kwargs() if pg else {}

    B = 1 << args.batch_log2
    S = args.bucket_bytes
    t_gen = time.perf_counter()
    nv, m_total, base_s, base_d, base_w = build_base(cfg, rank, world)
    # global degree hints (connectivity information known in advance)
    hints_t = torch.bincount(torch.from_numpy(base_s.astype(np.int64)).to(dev), minlength=nv)
    if pg:
        pg.all_reduce(hints_t, "sum")
    hints = hints_t.to(torch.int32).contiguous()
    del hints_t
    gen_s = time.perf_counter() - t_gen

    stream = torch.cuda.current_stream()
    ev = lambda: torch.cuda.Event(enable_timing=True)  # noqa: E731
    # warm-up on a tiny graph: loads the library's kernels (lazy module loading) so
    # the timed bulk build measures the build, not the first-launch overhead
    if world == 1:
        wg = Graph(1024, bucket_bytes=S)
        ws_, wd_, ww_ = (torch.from_numpy(x).to(dev) for x in wl.uniform_edges(1, 1, 4096, 1024))
        wg.insert_edges(ws_, wd_, ww_, count=True)
        wg.query_edges(ws_, wd_)
        wg.delete_edges(ws_, wd_, count=True)
        wg.delete_vertices(ws_[:16])
        wg.close()
    # ---- bulk build: create from hints + one insert of all edges
    torch.cuda.synchronize()
    if pg:
        pg.barrier()
    c0, c1, c2 = ev(), ev(), ev()
    c0.record()
    g = Graph(nv, hints, bucket_bytes=S, load_factor=args.load_factor, rank=rank, nranks=world,
              set_variant=args.variant == "set", **gkw)
    c1.record()
    bs = torch.from_numpy(base_s).to(dev)
    bd = torch.from_numpy(base_d).to(dev)
    bw = torch.from_numpy(base_w).to(dev)
    torch.cuda.synchronize()
    c1b = ev()
    g.profile_enable(True)  # kernel-side time of the build (events around the library's kernels)
    c1b.record()
    added = g.insert_edges(bs, bd, bw, count=True)
    c2.record()
    torch.cuda.synchronize()
    bprof = g.profile_read()
    g.profile_enable(False)
    # insert_ms is the whole call (first-touch reservation of the overflow pool and the
    # count read-back included); insert_kernel_ms is the insert kernel's own time
    bulk = {"create_ms": c0.elapsed_time(c1), "insert_ms": c1b.elapsed_time(c2),
            "insert_kernel_ms": bprof["kernel_ms"]["insert"],
            "insert_kernel_launches": bprof["kernel_launches"]["insert"],
            "edges": int(m_total), "unique_added": int(added)}
    bulk["M_edges_s"] = m_total / world / (bulk["insert_ms"] * 1e3)
    # the same build from src-sorted input: each table is then
    # filled by consecutive ops (the sort itself is input preparation, not timed)
    if world == 1 and not args.no_sorted_build:
        order = torch.argsort(bs.to(torch.int64), stable=True)
        i32 = torch.int32  # (uint32 tensors have no CUDA gather)
        ss_, sd_, sw_ = (x.view(i32)[order].view(torch.uint32).contiguous() for x in (bs, bd, bw))
        del order
        g2 = Graph(nv, hints, bucket_bytes=S, load_factor=args.load_factor,
                   set_variant=args.variant == "set")
        torch.cuda.synchronize()
        d0, d1 = ev(), ev()
        g2.profile_enable(True)
        d0.record()
        added2 = g2.insert_edges(ss_, sd_, sw_, count=True)
        d1.record()
        torch.cuda.synchronize()
        assert added2 == added, (added2, added)
        bulk["sorted_insert_ms"] = d0.elapsed_time(d1)
        bulk["sorted_insert_kernel_ms"] = g2.profile_read()["kernel_ms"]["insert"]
        bulk["sorted_M_edges_s"] = m_total / (bulk["sorted_insert_ms"] * 1e3)
        g2.close()
        del ss_, sd_, sw_
    del bs, bd, bw
    st0 = g.stats()

    flush = L2Flush(dev)
    # degree-adaptive layout (S = 0): the model uses the mean bytes of a linked bucket
    Sm = S or st0["table_bytes"] / max(1, st0["base_buckets"] + st0["overflow_buckets"])
    mb = model_bytes(Sm)

    def to_dev(a):
        return torch.from_numpy(np.ascontiguousarray(a)).to(dev, non_blocking=False)

    found = torch.empty(B, dtype=torch.uint8, device=dev)
    qw = torch.empty(B, dtype=torch.uint32, device=dev)
    host_batches = []
    tot = {"insert": 0.0, "query": 0.0, "delete": 0.0}
    per_step = {"insert": [], "query": [], "delete": []}  # for the median
    kbytes = {"insert": 0, "query": 0, "delete": 0}
    counts = {"added": 0, "removed": 0, "found": 0, "selfloops": 0}
    clock = None
    launches = 0
    kernel = None
    cleanup = {"ms": 0.0, "launches": 0, "all": 0}  # the untimed deletes' share of the profile
    for step in range(args.warmup + args.steps):
        timed = step >= args.warmup
        (s, d, w), (qs, qd), (xs, xd) = step_batch(cfg, nv, B, step, rank, world,
                                                   (None, m_total, (base_s, base_d)))
        if rank == 0 and len(host_batches) < 4:
            host_batches.append(((s, d, w), (qs, qd), (xs, xd)))
        S_, D_, W_, QS, QD, XS, XD = (to_dev(x) for x in (s, d, w, qs, qd, xs, xd))
        loops_i = int((s == d).sum())
        loops_q = int((qs == qd).sum())
        loops_x = int((xs == xd).sum())
        if timed and step == args.warmup:
            torch.cuda.synchronize()
            if pg:
                pg.barrier()
            g.profile_enable(True)
            clock = ClockSampler(local if "CUDA_VISIBLE_DEVICES" not in os.environ
                                 else os.environ["CUDA_VISIBLE_DEVICES"].split(",")[local])
        e = [ev() for _ in range(6)]
        torch.cuda.synchronize()
        if pg:
            pg.barrier()
        flush()
        e[0].record()
        g.insert_edges(S_, D_, W_)
        e[1].record()
        n_added = g.profile_read()["last_count"] if timed else 0
        flush()
        e[2].record()
        g.query_edges(QS, QD, found_out=found, weight_out=qw)
        e[3].record()
        n_found = int(found.sum().item()) if timed else 0
        flush()
        e[4].record()
        g.delete_edges(XS, XD)
        e[5].record()
        torch.cuda.synchronize()
        if timed:
            n_removed = g.profile_read()["last_count"]
        # untimed: the other half of this step's inserted edges, so every step starts
        # from the bulk-built graph (not counted as work, outside the events; its
        # kernel time is taken out of the profile below)
        p0 = g.profile_read() if timed else None
        g.delete_edges(S_[B // 2:], D_[B // 2:])
        torch.cuda.synchronize()
        if timed:
            p1 = g.profile_read()
            cleanup["ms"] += p1["kernel_ms"]["delete"] - p0["kernel_ms"]["delete"]
            cleanup["launches"] += p1["kernel_launches"]["delete"] - p0["kernel_launches"]["delete"]
            cleanup["all"] += p1["launches"] - p0["launches"]
        if timed:
            for k, (x, y) in zip(("insert", "query", "delete"), ((0, 1), (2, 3), (4, 5))):
                ms = e[x].elapsed_time(e[y])
                tot[k] += ms
                per_step[k].append(ms)
            counts["added"] += n_added
            counts["removed"] += n_removed
            counts["found"] += n_found
            counts["selfloops"] += loops_i
            kbytes["insert"] += (n_added * mb["insert_new"] + (B - loops_i - n_added) *
                                 mb["insert_replace"] + loops_i * mb["selfloop_insert"])
            kbytes["delete"] += (n_removed * mb["delete_hit"] + (B - loops_x - n_removed) *
                                 mb["delete_miss"] + loops_x * mb["selfloop_other"])
            kbytes["query"] += (B - loops_q) * mb["query"] + loops_q * mb["selfloop_other"]
    prof = g.profile_read()
    clocks = clock.stop() if clock else None
    prof["kernel_ms"]["delete"] -= cleanup["ms"]
    prof["kernel_launches"]["delete"] -= cleanup["launches"]
    launches = prof["launches"] - cleanup["all"]
    g.profile_enable(False)

    # max over ranks of the per-op device times (weak scaling: every rank does B per op)
    times = torch.tensor([tot["insert"], tot["query"], tot["delete"]], dtype=torch.float64,
                         device=dev)
    kms = torch.tensor([prof["kernel_ms"]["insert"], prof["kernel_ms"]["query"],
                        prof["kernel_ms"]["delete"]], dtype=torch.float64, device=dev)
    if pg:
        pg.all_reduce(times, "max")
        pg.all_reduce(kms, "max")
    t_ins, t_q, t_del = times.tolist()
    total_ms = t_ins + t_q + t_del
    K = args.steps
    ops_total = 3 * B * K * world
    value = ops_total / (total_ms * 1e3)

    # ---- roofline of the dominant kernel (model bytes / its event-timed duration)
    peak, peak_src = load_peaks()
    kinds = ["insert", "query", "delete"]
    kmsl = kms.tolist()
    dom = max(range(3), key=lambda i: kmsl[i])
    dk = kinds[dom]
    n_launch = max(1, prof["kernel_launches"][dk])
    achieved = kbytes[dk] / (kmsl[dom] * 1e-3) / 1e9
    traffic = None
    tpath = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if os.path.exists(tpath):
        try:
            tj = json.load(open(tpath))
            ent = tj.get(f"{args.config}/{dk}/b{args.batch_log2}/s{S}") if S else None
            if ent:
                traffic = ent["dram_bytes_per_launch"]
        except (ValueError, KeyError):
            traffic = None
    roofline = {"bound": "hbm", "kernel": f"k_edges<{S // 16 if S else 'adaptive'},{dk}>",
                "achieved": achieved,
                "peak": peak, "unit": "GB/s", "frac": achieved / peak, "traffic": traffic,
                "algorithmic_bytes_per_launch": kbytes[dk] / n_launch,
                "peak_source": peak_src,
                "kernel_share_of_step": kmsl[dom] / total_ms if total_ms else None}
    # context beside the copy peak: the measured random-op ceiling of this GPU for the
    # dominant op's access pattern (tools/gather_ceiling.cu, profiles/r02/gather_ceiling.json):
    # insert/delete = 128-B gather + CAS + counter atomic, query = 128-B gather
    cpath = os.path.join(ROOT, "profiles", "r02", "gather_ceiling.json")
    if os.path.exists(cpath) and S == 128:
        try:
            cj = json.load(open(cpath))["G_ops_s_S128"]
            ceil = cj["read"] if dk == "query" else cj["read_cas8_counter"]
            gops = B * K / (kmsl[dom] * 1e6) if kmsl[dom] else 0.0  # per GPU
            roofline["random_op_ceiling"] = {
                "pattern": "128-B gather" if dk == "query" else "128-B gather + 64-bit CAS + counter atomic",
                "G_ops_s": ceil, "achieved_G_ops_s": gops,
                "frac": gops / ceil if ceil else None,
                "source": "tools/gather_ceiling.cu (profiles/r02/gather_ceiling.json)"}
        except (ValueError, KeyError):
            pass
    ops = {}
    for i, k in enumerate(kinds):
        t = [t_ins, t_q, t_del][i]
        ops[k] = {"M_edges_s": B * K * world / (t * 1e3), "ms_per_batch": t / K,
                  "ms_per_batch_median": statistics.median(per_step[k]) if per_step[k] else None,
                  "kernel_ms_per_batch": kmsl[i] / K,
                  "kernel_GBs": kbytes[k] / (kmsl[i] * 1e-3) / 1e9 if kmsl[i] else None}
    ops["insert"]["added_per_batch"] = counts["added"] / K
    ops["delete"]["removed_per_batch"] = counts["removed"] / K
    ops["delete"]["hit_rate"] = counts["removed"] / (K * B)
    ops["delete"]["batch"] = "half of the step's inserted edges + half uniform pairs"
    ops["query"]["found_per_batch"] = counts["found"] / K

    # ---- e2e: same steps through the public API with pinned HOST buffers
    e2e = None
    if not args.no_e2e:
        E = min(3, K)
        e2e_ms = 0.0
        e2e_wall = {}
        # the caller's pinned batch and result buffers, allocated once and refilled with
        # every step's data outside the timed region (as a streaming client would)
        hf = torch.empty(B, dtype=torch.uint8).pin_memory()
        hqw = torch.empty(B, dtype=torch.uint32).pin_memory()
        hin = [torch.empty(B, dtype=torch.int32).pin_memory() for _ in range(7)]
        for step in range(-1, E):  # step -1: untimed warm-up (staging buffers, pinning)
            (s, d, w), (qs, qd), (xs, xd) = step_batch(cfg, nv, B, 100 + step, rank, world,
                                                       (None, m_total, (base_s, base_d)))
            for h, x in zip(hin, (s, d, w, qs, qd, xs, xd)):  # this step's batch, pinned
                h.numpy()[:] = np.ascontiguousarray(x, np.uint32).view(np.int32)
            hs, hd, hw, hq, hqd, hxs, hxd = hin
            torch.cuda.synchronize()
            if pg:
                pg.barrier()
            flush()
            a, b = ev(), ev()
            t0 = time.perf_counter()
            a.record()
            g.insert_edges(hs, hd, hw)
            t1 = time.perf_counter()
            g.query_edges(hq, hqd, found_out=hf, weight_out=hqw)
            t2 = time.perf_counter()
            g.delete_edges(hxs, hxd)
            t3 = time.perf_counter()
            b.record()
            torch.cuda.synchronize()
            t4 = time.perf_counter()
            g.delete_edges(S_cleanup := torch.from_numpy(s[B // 2:]).to(dev),
                           torch.from_numpy(d[B // 2:]).to(dev))  # untimed, as above
            del S_cleanup
            torch.cuda.synchronize()
            if step >= 0:
                e2e_ms += a.elapsed_time(b)
                for k, dt in zip(("insert", "query", "delete", "tail"), (t1 - t0, t2 - t1, t3 - t2, t4 - t3)):
                    e2e_wall[k] = e2e_wall.get(k, 0.0) + 1e3 * dt
        t = torch.tensor([e2e_ms], dtype=torch.float64, device=dev)
        if pg:
            pg.all_reduce(t, "max")
        e2e_ms = t.item()
        e2e = {"value": 3 * B * E * world / (e2e_ms * 1e3), "unit": UNIT,
               "h2d_bytes_per_step": B * (12 + 8 + 8), "d2h_bytes_per_step": B * 5 + 3 * 64,
               "steps": E, "host_ms_per_call": {k: v / E for k, v in e2e_wall.items()}}

    # ---- cfg3: road growth — insert, then delete, batches of held-out lattice edges
    # (edges of the grid the generator did not keep), 2^20 and 2^22
    lattice = None
    if cfg["kind"] == "grid" and world == 1:
        hs_all, hd_all = wl.grid_heldout_edges(cfg["seed"], cfg["rows"], cfg["cols"], cfg["p"])
        lattice = {"held_out_edges": int(hs_all.size)}
        for lb in (20, 22):
            idx = wl.uniform_index(cfg["seed"], 424242 + lb, 1 << lb, hs_all.size)
            HS, HD = to_dev(hs_all[idx]), to_dev(hd_all[idx])
            HW = to_dev(wl.weights(cfg["seed"], 525252 + lb, 1 << lb))
            r = {}
            for name, fn in (("insert", lambda: g.insert_edges(HS, HD, HW)),
                             ("delete", lambda: g.delete_edges(HS, HD))):
                torch.cuda.synchronize()
                flush()
                a, b = ev(), ev()
                a.record()
                fn()
                b.record()
                torch.cuda.synchronize()
                r[name + "_M_edges_s"] = (1 << lb) / (a.elapsed_time(b) * 1e3)
            lattice[f"b{lb}"] = r
        del hs_all, hd_all

    # ---- vertex deletion (a9) on the built graph: 2^12 vertices (directed sweep)
    vdel = None
    if not args.no_vdel:
        ids = torch.from_numpy(wl.uniform_u32(cfg["seed"], 31337, 4096, nv, offset=rank * 4096)).to(dev)
        # untimed warm-up batch (scratch buffers), different IDs
        g.delete_vertices(torch.from_numpy(wl.uniform_u32(cfg["seed"], 31338, 64, nv,
                                                          offset=rank * 64)).to(dev))
        torch.cuda.synchronize()
        if pg:
            pg.barrier()
        flush()
        a, b = ev(), ev()
        a.record()
        g.delete_vertices(ids)
        b.record()
        torch.cuda.synchronize()
        vms = a.elapsed_time(b)
        vdel = {"ids_per_gpu": 4096, "ms": vms, "M_vertices_s": 4096 * world / (vms * 1e3),
                "pool_bytes_swept": st0["bump_bytes"]}

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cpu = cpu_baseline(cfg, nv, base_s, base_d, base_w, host_batches)

    line = {
        "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": K,
        "warmup": args.warmup, "ms_per_step": total_ms / K, "higher_is_better": True,
        "scaling": "weak", "vs_baseline": None, "dtype": "u32",
        "data": "synthetic (seeded counter-based generators, workloads/gen.c)",
        "config": config_block(cfg, args, nv, m_total, B, world),
        "ops": ops, "bulk_build": bulk, "vertex_deletion": vdel, "lattice_growth": lattice,
        "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": launches,
        "clocks": clocks,
        "graph": {"live_pairs": st0["live_pairs"], "base_buckets": st0["base_buckets"],
                  "overflow_buckets": st0["overflow_buckets"], "max_chain": st0["max_chain"],
                  "load_factor": st0["load_factor"], "pool_bytes": st0["pool_bytes"]},
        "gen_s": gen_s,
    }
    if rank == 0:
        print(json.dumps(line), flush=True)
    g.close()
    if pg:
        pg.close()
    return 0


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--config", choices=sorted(CONFIGS), default="cfg2")
    ap.add_argument("--batch-log2", type=int, default=24)
    ap.add_argument("--bucket-bytes", type=int, default=None,
                    help="bucket bytes (32/64/128); default 128, 64 for cfg5 (TC on the set variant)")
    ap.add_argument("--load-factor", type=float, default=0.7)
    ap.add_argument("--variant", choices=["map", "set"], default=None,
                    help="per-vertex table variant (P:L366-370); default map, set for cfg5 (TC)")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-vdel", action="store_true")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-sorted-build", action="store_true",
                    help="skip the second bulk build from src-sorted input")
    ap.add_argument("--inproc", type=int, default=0,
                    help="dry run of the N-rank path: N rank threads of this process over an "
                         "in-process rank group on the visible GPUs (not a scaling measurement)")
    args = ap.parse_args()
    cfg = CONFIGS[args.config]
    if args.bucket_bytes is None:  # TC probes whole buckets: 64-B set buckets (14 keys) move half the bytes
        args.bucket_bytes = 64 if cfg.get("tc") and args.variant != "map" else 128
    if args.impl == "reference":
        return run_reference(args, cfg)
    if cfg.get("stream"):
        import bench_stream
        fn = bench_stream.run_mixed
    elif cfg.get("tc"):
        import bench_stream
        fn = bench_stream.run_tc
    else:
        fn = run_ours
    if args.inproc > 1:
        return run_inproc(args, fn)
    return fn(args, cfg)


if __name__ == "__main__":
    sys.exit(main())
