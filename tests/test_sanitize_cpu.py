"""Host code under AddressSanitizer + UndefinedBehaviorSanitizer.

* The oracle (oracle/*.c, plain C, test infrastructure) linked into tests/sanitize/
  oracle_driver.c, which runs every entry point on small and degenerate shapes.
* The C ABI's host logic (sepconv_api/band/host/tune/dispatch.cpp, and the host side of
  sor.cu, bs.cu, sepconv_util.cu) instrumented and linked into tests/sanitize/abi_driver.cpp
  with tests/sanitize/kernel_stubs.cpp standing in for the kernel translation units:
  validation of every entry point, the band partitions, SELECT over random selectors and,
  where a GPU exists, plan creation against fuzzed tuning-cache files.
Both are built with -fsanitize=address,undefined -fno-sanitize-recover=all: any report
aborts the driver.  Objects are cached under build/sanitize (rebuilt when a source changes)."""
import concurrent.futures as cf
import glob
import os
import shutil
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
CSRC = os.path.join(ROOT, "paper_conf_asplos_phothilimthanaara13_b200", "csrc")
SAN = os.path.join(ROOT, "tests", "sanitize")
OUT = os.path.join(ROOT, "build", "sanitize")
FLAGS = ["-O1", "-g", "-fsanitize=address,undefined", "-fno-sanitize-recover=all", "-fno-omit-frame-pointer"]
CUDA = "/usr/local/cuda"
ENV = dict(os.environ, ASAN_OPTIONS="protect_shadow_gap=0:detect_leaks=0:abort_on_error=0",
           UBSAN_OPTIONS="print_stacktrace=1:halt_on_error=1")


def _stale(obj, deps):
    return not os.path.exists(obj) or any(os.path.getmtime(d) > os.path.getmtime(obj) for d in deps)


def _run(cmd):
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError("%s\n%s\n%s" % (" ".join(cmd), r.stdout[-3000:], r.stderr[-3000:]))


def _compile(src, headers):
    obj = os.path.join(OUT, os.path.basename(src) + ".o")
    if not _stale(obj, [src] + headers):
        return obj
    inc = ["-I" + os.path.join(ROOT, "include"), "-I" + CSRC]
    if src.endswith(".cu"):
        nvcc = shutil.which("nvcc") or os.path.join(CUDA, "bin", "nvcc")
        xc = []                          # nvcc splits -Xcompiler values on commas: one flag each
        for f in ["-fsanitize=address", "-fsanitize=undefined", "-fno-sanitize-recover=all", "-fno-omit-frame-pointer"]:
            xc += ["-Xcompiler", f]
        _run([nvcc, "-std=c++17", "-O1", "-g", "-gencode", "arch=compute_100a,code=sm_100a", *xc, *inc, "-c", src,
              "-o", obj])
    else:
        _run(["g++", "-std=c++17", *FLAGS, "-I" + os.path.join(CUDA, "include"), *inc, "-c", src, "-o", obj])
    return obj


@pytest.fixture(scope="module")
def drivers():
    if not shutil.which("gcc") or not shutil.which("g++"):
        pytest.skip("no host compiler")
    os.makedirs(OUT, exist_ok=True)
    oracle_src = [os.path.join(ROOT, "oracle", f) for f in ("oracle.c", "poisson.c", "blackscholes.c")]
    oracle_bin = os.path.join(OUT, "oracle_driver")
    if _stale(oracle_bin, oracle_src + [os.path.join(SAN, "oracle_driver.c")]):
        _run(["gcc", "-std=c11", *FLAGS, "-pthread", os.path.join(SAN, "oracle_driver.c"), *oracle_src, "-lm",
              "-o", oracle_bin])
    headers = glob.glob(os.path.join(CSRC, "*.h")) + glob.glob(os.path.join(CSRC, "*.cuh")) + \
        glob.glob(os.path.join(ROOT, "include", "*.h"))
    host = [os.path.join(CSRC, f) for f in ("sepconv_api.cpp", "sepconv_band.cpp", "sepconv_host.cpp",
                                            "sepconv_tune.cpp", "sepconv_dispatch.cpp", "sor.cu", "bs.cu",
                                            "sepconv_util.cu")]
    host += [os.path.join(SAN, "kernel_stubs.cpp"), os.path.join(SAN, "abi_driver.cpp")]
    with cf.ThreadPoolExecutor(max(1, min(len(host), os.cpu_count() or 4))) as ex:
        objs = list(ex.map(lambda s: _compile(s, headers), host))
    abi_bin = os.path.join(OUT, "abi_driver")
    if _stale(abi_bin, objs):
        _run(["g++", *FLAGS, *objs, "-L" + os.path.join(CUDA, "lib64"), "-lcudart_static", "-ldl", "-lpthread", "-lrt",
              "-o", abi_bin])
    return oracle_bin, abi_bin


def _check(binary):
    r = subprocess.run([binary], capture_output=True, text=True, timeout=600, env=ENV, cwd=OUT)
    report = r.stdout[-2000:] + r.stderr[-4000:]
    assert r.returncode == 0, report
    assert "runtime error" not in r.stderr and "AddressSanitizer" not in r.stderr, report
    return r.stdout


def test_oracle_under_asan_ubsan(drivers):
    assert "oracle sanitize ok" in _check(drivers[0])


def test_c_abi_host_logic_under_asan_ubsan(drivers):
    assert "abi sanitize ok" in _check(drivers[1])
