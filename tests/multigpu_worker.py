"""torchrun worker: P ranks, one GPU each, graph sharded by source vertex (owner
u mod P) over NCCL.  Every rank runs the shared multi-rank stream
(``tests/multirank.py``: uneven slices, a batch rejected on one rank, out-of-range
queries, deletes, vertex deletion and insertion, undirected mirror ops) once per
exchange (fused NVLink windows, copy exchange) and per mode (directed, undirected);
rank 0 gathers the records and checks them against the unsharded oracle.

    python -m torch.distributed.run --nproc-per-node P --master-addr 127.0.0.1 \\
        tests/multigpu_worker.py
"""
import os
import sys

import numpy as np
import torch
import torch.distributed as dist

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

from paper_conf_ipps_awadapo20_b200 import Graph, get_unique_id  # noqa: E402
from tests import multirank  # noqa: E402


def main():
    rank, P = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    local = int(os.environ["LOCAL_RANK"])
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist.init_process_group("nccl", device_id=dev)
    to_dev = lambda a: torch.from_numpy(np.ascontiguousarray(a, np.uint32)).to(dev)  # noqa: E731
    for directed in (True, False):
        for copy_exchange in (False, True):
            obj = [get_unique_id() if rank == 0 else None]
            dist.broadcast_object_list(obj, src=0)
            g = Graph(multirank.NV0, rank=rank, nranks=P, nccl_unique_id=obj[0],
                      directed=directed, copy_exchange=copy_exchange)
            recs = multirank.run_rank(g, rank, P, to_dev)
            out = [None] * P if rank == 0 else None
            dist.gather_object(recs, out, dst=0)
            if rank == 0:
                ex = multirank.check(out, P, directed=directed)
                print(f"MULTIGPU OK P={P} directed={directed} copy={copy_exchange} "
                      f"exchange={ex}", flush=True)
            torch.cuda.synchronize()
            dist.barrier()
            g.close()
    dist.barrier()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
