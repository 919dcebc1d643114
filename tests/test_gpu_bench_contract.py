"""bench.py keeps the driver's JSON-line contract on a B200 (a short run of each workload):
metric / value / unit, n_gpus, steps, warmup, ms_per_step, higher_is_better, scaling, dtype,
config.workload and config.l2, roofline {bound, achieved, peak, unit, frac, traffic},
e2e {value, unit, h2d/d2h bytes}, gpu_launches > 0 and the clocks sample.  -m gpu only."""
import json
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def run(*args):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--steps", "3", "--warmup", "3",
                          "--no-cpu-baseline", *args], capture_output=True, text=True, timeout=900, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-3000:]
    lines = [ln for ln in out.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, out.stdout
    return json.loads(lines[0])


def check_common(d, unit):
    for key in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better",
                "scaling", "dtype", "data", "config", "roofline", "e2e", "gpu_launches", "clocks"):
        assert key in d, key
    assert d["unit"] == unit and d["value"] > 0 and d["n_gpus"] == 1 and d["steps"] == 3 and d["warmup"] == 3
    assert d["higher_is_better"] is True and d["gpu_launches"] > 0
    assert d["config"]["workload"] and d["config"]["l2"]
    r = d["roofline"]
    assert r["bound"] == "hbm" and r["unit"] == "GB/s" and r["peak"] > 0
    assert abs(r["frac"] - r["achieved"] / r["peak"]) < 1e-9
    e = d["e2e"]
    assert e["value"] > 0 and e["h2d_bytes_per_step"] > 0 and e["d2h_bytes_per_step"] > 0
    assert "sm_mhz" in d["clocks"] and "reasons" in d["clocks"]


def test_image_workload_line():
    d = run("--size", "2048", "--widths", "3,17")
    check_common(d, "Mpixels/s")
    assert set(d["per_width"]) == {"3", "17"} and d["config"]["widths"] == [3, 17]
    assert "flushed" in d["config"]["l2"]                      # 33 MB fits in 2 x L2
    # launches per pass follow the tuner's pick on this box (never assume one): 2 for the
    # unfused pair (ConvolveRows + ConvolveColumns), 1 for every single-kernel candidate
    per_pass = sum(2 if w["variant"].startswith("sep-unfused") else 1 for w in d["per_width"].values())
    assert d["gpu_launches"] == per_pass * d["steps"], (d["gpu_launches"], d["per_width"])


def test_poisson_and_black_scholes_lines():
    check_common(run("--workload", "poisson", "--size", "1024", "--sor-iters", "8"), "Mcell-it/s")
    check_common(run("--workload", "blackscholes", "--options", "1000000"), "Moptions/s")
