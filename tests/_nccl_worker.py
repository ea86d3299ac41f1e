"""Worker for tests/test_gpu_nccl.py (launched by torch.distributed.run): the
partitioned COUNT path over a real NCCL communicator vs the oracle."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import graphgen as G  # noqa: E402
import oracle as O  # noqa: E402
import paper_conf_ipps_osamatybo19_b200 as gcb  # noqa: E402
from paper_conf_ipps_osamatybo19_b200 import dist as gdist  # noqa: E402


def main():
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    local = int(os.environ.get("LOCAL_RANK", 0))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist.init_process_group("nccl", device_id=dev)
    scale = int(os.environ.get("GC_TEST_SCALE", "14"))
    (ro, ci), h, n, nnz = gdist.build_partitioned_rmat(scale, 16, 1, rank, world, dev)
    ref, R, nk = O.color_maxmin(G.rmat(scale, 16, seed=1), 1, with_stats=True)
    for mode in (gcb.MODE_AUTO, gcb.MODE_SWEEP):
        out = torch.empty(n, dtype=torch.int32, device=dev)
        _, k, st = h.color(1, gcb.MAXMIN, out, stats=True, mode=mode, frontier_cap=1 << 16)
        C = out.cpu().numpy().view(np.uint32)
        assert (C == ref).all(), (rank, mode)
        assert st.rounds == R and st.frontier_sizes == nk and k == O.count_colors(ref)
    h.close()
    dist.barrier()
    dist.destroy_process_group()
    print(f"rank {rank}/{world}: partitioned colouring over NCCL equals the oracle", flush=True)


if __name__ == "__main__":
    main()
