"""Multi-process (gloo, CPU) test of the Poisson SOR row-band protocol sor_band_iterate
implements: the partition from the C library's sor_band (even band
starts), `halo` ghost rows on each side with a neighbour, passes of depth T = halo/2 that
treat the ghost rows as fixed, and after every pass the first/last `halo` owned rows sent
to the neighbours.  The fixed-order float32 oracle stands in for the kernels; the owned
rows, concatenated, must equal the whole-grid oracle bit for bit."""
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


def _worker(rank, world, port, N, M, halo, iters, result_q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        from paper_conf_asplos_phothilimthanaara13_b200 import sor, synth

        r0, rows, a0, arows = sor.band(N, world, rank, halo)
        x, b = synth.poisson_problem(N, M, seed=91, guess="uniform")
        u = np.ascontiguousarray(x[a0:a0 + arows])
        bb = np.ascontiguousarray(b[a0:a0 + arows])
        h_top = r0 - a0
        h_bot = a0 + arows - (r0 + rows)
        T = halo // 2
        omega = 1.7
        left = iters
        while left > 0:
            t = min(T, left)
            u = oracle.sor_rb_f32(u, bb, omega, t)            # ghost rows fixed, as in the kernels
            ops, recvs = [], []
            if rank > 0:
                ops.append(dist.P2POp(dist.isend, torch.from_numpy(u[h_top:h_top + halo].copy()), rank - 1))
                rt = torch.empty((halo, M), dtype=torch.float32)
                ops.append(dist.P2POp(dist.irecv, rt, rank - 1))
                recvs.append((0, rt))
            if rank < world - 1:
                n = u.shape[0]
                ops.append(dist.P2POp(dist.isend, torch.from_numpy(u[n - h_bot - halo:n - h_bot].copy()), rank + 1))
                rb = torch.empty((halo, M), dtype=torch.float32)
                ops.append(dist.P2POp(dist.irecv, rb, rank + 1))
                recvs.append((n - halo, rb))
            for w in (dist.batch_isend_irecv(ops) if ops else []):
                w.wait()
            for off, rt in recvs:
                u[off:off + halo] = rt.numpy()
            left -= t
        parts = [None] * world
        dist.all_gather_object(parts, (r0, u[h_top:h_top + rows]))
        if rank == 0:
            want = oracle.sor_rb_f32(x, b, omega, iters)
            got = np.concatenate([o for _, o in sorted(parts, key=lambda p: p[0])], axis=0)
            result_q.put(bool(np.array_equal(got, want)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,N,M,halo,iters", [(2, 40, 23, 4, 7), (3, 61, 30, 6, 9), (2, 33, 17, 2, 3)])
def test_sor_row_band_protocol(world, N, M, halo, iters):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, N, M, halo, iters, q)) for r in range(world)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(timeout=120)
    assert all(p.exitcode == 0 for p in procs), [p.exitcode for p in procs]
    assert q.get(timeout=10) is True
