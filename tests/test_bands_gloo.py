"""Multi-process (gloo, CPU) test of the row-band protocol sepconv_run_band implements:
partition from the C library's sepconv_band, owned rows per rank, the one-sided K-1
row halo sent by rank g to rank g-1 (windows extend to +y), each band
convolved on its own (the oracle stands in for the kernels here), and the
concatenated bands equal to the whole-image result bit for bit."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    return port


def _worker(rank, world, port, H, W, K, result_q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
        from paper_conf_asplos_phothilimthanaara13_b200 import synth

        r0, rows, owned, alloc = sc.band(H, K, world, rank)
        band = np.full((alloc, W), np.nan, np.float32)
        band[:owned] = synth.uniform_image(H, W, seed=77, rows=(r0, r0 + owned))
        halo = K - 1
        t = torch.from_numpy(band)
        ops = []
        if halo and rank > 0:
            ops.append(dist.P2POp(dist.isend, t[:halo].contiguous(), rank - 1))
        recv = torch.empty((halo, W), dtype=torch.float32)
        if halo and rank < world - 1:
            ops.append(dist.P2POp(dist.irecv, recv, rank + 1))
        for w in (dist.batch_isend_irecv(ops) if ops else []):
            w.wait()
        if halo and rank < world - 1:
            band[rows:rows + halo] = recv.numpy()
        assert not np.any(np.isnan(band)), "halo rows missing"
        k = synth.random_kernel(K, seed=K, signed=True)
        out = oracle.convolve2d(band, k)
        assert out.shape == (rows, W - K + 1)
        parts = [None] * world
        dist.all_gather_object(parts, (r0, out))
        if rank == 0:
            full = synth.uniform_image(H, W, seed=77)
            want = oracle.convolve2d(full, k)
            got = np.concatenate([o for _, o in sorted(parts, key=lambda p: p[0])], axis=0)
            result_q.put(bool(np.array_equal(got, want)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,H,W,K", [(2, 61, 40, 5), (2, 64, 33, 17), (2, 20, 9, 1), (3, 100, 21, 9)])
def test_row_band_halo_protocol(world, H, W, K):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, H, W, K, q)) for r in range(world)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(timeout=120)
    assert all(p.exitcode == 0 for p in procs), [p.exitcode for p in procs]
    assert q.get(timeout=10) is True
