"""bench.py's multi-GPU launcher on the GPU-less dev box.  `python bench.py --gpus N` outside
torchrun must start N ranks itself (never silently measure one GPU), and must refuse when the
node has fewer devices or WORLD_SIZE disagrees with --gpus.  --dry-run runs the image
workload's band partition and (K-1)-row halo exchange on gloo with no convolution, so the
spawn, rank plumbing and exchange protocol are covered here (
DESIGN.md R18)."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _bench(*args, env=None, timeout=600):
    e = dict(os.environ)
    for k in ("WORLD_SIZE", "RANK", "LOCAL_RANK", "MASTER_ADDR", "MASTER_PORT"):
        e.pop(k, None)
    e.update(env or {})
    return subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True,
                          text=True, timeout=timeout, cwd=ROOT, env=e)


@pytest.mark.parametrize("n", [2, 3])
def test_gpus_n_spawns_n_ranks(n):
    out = _bench("--gpus", str(n), "--dry-run", "--size", "1024", "--widths", "3,17")
    assert out.returncode == 0, out.stderr[-3000:]
    lines = [ln for ln in out.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, out.stdout                     # rank 0 alone prints
    d = json.loads(lines[0])
    assert d["n_gpus"] == n and d["dry_run"] is True and d["halo_exchange_ok"] is True
    # every rank but the last receives K-1 rows of 1024 floats per width
    assert d["halo_bytes"] == (n - 1) * (2 + 16) * 1024 * 4
    assert "launching %d ranks" % n in out.stderr


def test_too_few_devices_is_an_error_not_a_one_gpu_run():
    out = _bench("--gpus", "2", "--steps", "1", "--warmup", "3", "--size", "256", "--widths", "3")
    assert out.returncode != 0
    assert "CUDA device" in out.stderr
    assert not [ln for ln in out.stdout.splitlines() if ln.startswith("{")]


def test_world_size_mismatch_is_an_error():
    out = _bench("--gpus", "4", "--steps", "1", "--warmup", "3", "--size", "256", "--widths", "3",
                 env={"WORLD_SIZE": "1", "RANK": "0", "LOCAL_RANK": "0"})
    assert out.returncode != 0 and "WORLD_SIZE=1" in out.stderr
