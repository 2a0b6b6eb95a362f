"""The P >= 2 router on ONE GPU (rows a2, a11 and §8(e) of SURVEY.md; -m gpu).

P host threads of this process act as the P ranks of a sharded graph through an
in-process rank group (``RankGroup`` / ``dg_group_create``): each thread owns a handle
(rank r of P) and a non-blocking stream, and makes every collective call with its own
slice.  The router's kernels run for real — per-block owner histogram and validation,
the counts all-gather, the fused partition + peer-store scatter into the owners'
windows with arrival counters and spin waits, the copy exchange (send buffers,
grouped send/recv), the answer return and the unpermute — only the transport is the
in-process one instead of NCCL.  ``tests/multirank.py`` holds the stream and the
oracle check (statuses, counts, every query answer, merged shard exports).
"""
import os
import threading

import numpy as np
import pytest
import torch

os.environ.setdefault("DG_GROUP_TIMEOUT_S", "60")

from tests import multirank  # noqa: E402

pytestmark = pytest.mark.gpu


def _run_group(P, directed=True, copy_exchange=False, env=None, bucket_bytes=128):
    from paper_conf_ipps_awadapo20_b200 import Graph, RankGroup
    old = {}
    for k, v in (env or {}).items():
        old[k] = os.environ.get(k)
        os.environ[k] = v
    try:
        grp = RankGroup(P)
        records = [None] * P
        errors = []
        dev = torch.device("cuda", 0)

        def rank_main(r):
            try:
                torch.cuda.set_device(0)
                s = torch.cuda.Stream(device=dev)
                with torch.cuda.stream(s):
                    g = Graph(multirank.NV0, rank=r, nranks=P, group=grp, directed=directed,
                              copy_exchange=copy_exchange, bucket_bytes=bucket_bytes, stream=s)
                    to_dev = lambda a: torch.from_numpy(np.ascontiguousarray(a, np.uint32)).to(dev)  # noqa: E731
                    records[r] = multirank.run_rank(g, r, P, to_dev)
                    torch.cuda.synchronize()
                    g.close()
            except BaseException as e:  # noqa: BLE001
                errors.append((r, repr(e)))

        th = [threading.Thread(target=rank_main, args=(r,)) for r in range(P)]
        for t in th:
            t.start()
        for t in th:
            t.join()
        assert not errors, errors
        return records
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


@pytest.mark.parametrize("P", [2, 3, 4, 8])
@pytest.mark.parametrize("exchange", ["fused", "copy"])
def test_router_p_ranks_directed(cuda_ok, P, exchange):
    recs = _run_group(P, directed=True, copy_exchange=exchange == "copy")
    ex = multirank.check(recs, P, directed=True)
    assert ex == [2 if exchange == "fused" else 1] * P  # dg_stats.exchange


@pytest.mark.parametrize("P", [2, 5])
@pytest.mark.parametrize("exchange", ["fused", "copy"])
def test_router_p_ranks_undirected(cuda_ok, P, exchange):
    """undirected mode: every op is mirrored before routing"""
    recs = _run_group(P, directed=False, copy_exchange=exchange == "copy")
    multirank.check(recs, P, directed=False)


def test_router_window_regrowth(cuda_ok):
    """windows start at 4,096 ops, so the first batches re-set them up (collective)"""
    recs = _run_group(4, env={"DG_ROUTER_WINDOW_OPS": "4096"})
    assert multirank.check(recs, 4) == [2] * 4


def test_router_window_regrowth_failure_falls_back(cuda_ok):
    """a failed window re-setup moves every rank to the copy exchange mid-batch
    (the batch must still be applied, not dropped)"""
    recs = _run_group(3, env={"DG_ROUTER_WINDOW_OPS": "4096", "DG_TEST_FUSED_REGROW_FAIL": "1"})
    assert multirank.check(recs, 3) == [1] * 3


def test_router_small_buckets(cuda_ok):
    recs = _run_group(3, bucket_bytes=32)
    multirank.check(recs, 3)


def test_router_single_rank_group(cuda_ok):
    """P = 1 through the in-process group (force_router): the router with itself"""
    from paper_conf_ipps_awadapo20_b200 import Graph, RankGroup
    from oracle import Oracle
    from tests.gpu_util import check_against_oracle, cuda
    import workloads as wl
    grp = RankGroup(1)
    g = Graph(5000, group=grp, force_router=True)
    o = Oracle(5000)
    s, d, w = wl.uniform_edges(5, 0, 30_000, 5000)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    check_against_oracle(g, o, "group P=1")
    assert g.stats()["exchange"] == 2
    g.close()
