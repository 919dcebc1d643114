"""bench.py --impl reference (the driver's reference arm: the CPU oracle on host cores) keeps the
JSON-line contract on the GPU-less dev box: one line, impl = reference, the CUDA arm's metric /
unit / workload string, a cpu_baseline describing the run and an e2e with zero copy bytes."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def run_bench(*extra):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--steps", "2",
                          "--warmup", "1", "--cpu-seconds", "0.3", *extra],
                         capture_output=True, text=True, timeout=600, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-2000:]
    lines = [ln for ln in out.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, out.stdout
    return json.loads(lines[0])


def test_reference_arm_image_line():
    d = run_bench("--size", "96", "--widths", "3,5")
    assert d["impl"] == "reference"
    assert d["unit"] == "Mpixels/s" and d["higher_is_better"] is True and d["value"] > 0
    assert d["metric"].startswith("output Mpixels/s")
    assert d["config"]["workload"] == "96x96 float32 image, kernel widths 3,5, one pass per width"
    assert d["config"]["widths"] == [3, 5]
    cb = d["cpu_baseline"]
    assert cb["kind"] == "oracle" and cb["cores"] >= 1 and cb["value"] == d["value"] and cb["sample"]
    assert d["e2e"] == {"value": d["value"], "unit": "Mpixels/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}
    # the CUDA arm's config key for key (the driver compares the two arms' configs)
    import argparse
    import bench
    args = argparse.Namespace(workload="image", variant="auto")
    assert d["config"] == bench.image_config(args, 1, 96, 96, 1, [3, 5], d["config"]["seed"],
                                             8 * 96 * 96 <= 2 * bench.l2_bytes_of())


def test_reference_arm_poisson_and_black_scholes_lines():
    import bench_bs
    import bench_poisson
    from bench import CleanFlush
    p = run_bench("--workload", "poisson", "--size", "64", "--sor-iters", "4")
    assert p["impl"] == "reference" and p["unit"] == "Mcell-it/s" and p["value"] > 0
    assert p["config"] == bench_poisson.sor_config(64, 4, 1, True, CleanFlush.LABEL)
    b = run_bench("--workload", "blackscholes", "--options", "1000")
    assert b["impl"] == "reference" and b["unit"] == "Moptions/s" and b["value"] > 0
    assert b["config"] == bench_bs.bs_config(1000, 1, True, CleanFlush.LABEL)


def test_reference_arm_other_ranks_exit_quietly():
    env = dict(os.environ, RANK="1", WORLD_SIZE="2", LOCAL_RANK="1")
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--steps", "1",
                          "--warmup", "0", "--size", "64", "--widths", "3"],
                         capture_output=True, text=True, timeout=300, cwd=ROOT, env=env)
    assert out.returncode == 0, out.stderr[-2000:]
    assert not [ln for ln in out.stdout.splitlines() if ln.startswith("{")]
