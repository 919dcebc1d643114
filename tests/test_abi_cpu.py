"""The C-ABI library without a GPU: it loads, exports every symbol include/sepconv.h
declares, validates arguments, and its pure-host band arithmetic matches the
oracle's independent partition (R18).  No compute calls."""
import os
import re

import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
from paper_conf_asplos_phothilimthanaara13_b200 import bs, sor

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared():
    hdr = open(os.path.join(ROOT, "include", "sepconv.h")).read()
    return sorted(set(re.findall(r"\b(sepconv_[a-z0-9_]+)\s*\(", hdr)))


def test_library_exports_every_declared_symbol():
    L = sc.lib()
    declared = _declared()
    assert len(declared) >= 19
    for name in declared:
        assert hasattr(L, name), name
    assert sorted(sc.exported_symbols()) == declared


def test_library_exports_every_sor_symbol():
    hdr = open(os.path.join(ROOT, "include", "sor.h")).read()
    declared = sorted(set(re.findall(r"\b(sor_[a-z_]+)\s*\(", hdr)))
    L = sor.lib()
    assert len(declared) == 13
    for name in declared:
        assert hasattr(L, name), name
    assert sorted(sor.exported_symbols()) == declared


def test_library_exports_every_bs_symbol():
    hdr = open(os.path.join(ROOT, "include", "bs.h")).read()
    declared = sorted(set(re.findall(r"\b(bs_[a-z_]+)\s*\(", hdr)))
    L = bs.lib()
    assert declared == sorted(bs.exported_symbols())
    for name in declared:
        assert hasattr(L, name), name


def test_bs_validation_before_device():
    import numpy as np
    a = np.ones(8, np.float32)
    with pytest.raises(sc.SepconvError) as ei:
        bs.price(a.ctypes.data, a.ctypes.data, a.ctypes.data, 0.02, -1.0, 0, 0, n=8, stream=0)
    assert ei.value.code == "E_INVALID"


def test_sor_plan_validation_and_no_device():
    with pytest.raises(sc.SepconvError) as ei:
        sor.SorPlan(0, 5)
    assert ei.value.code == "E_INVALID"
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available():
        with pytest.raises(sc.SepconvError) as ei:
            sor.SorPlan(64, 64)
        assert ei.value.code == "E_UNSUPPORTED"


def test_status_strings_and_version():
    L = sc.lib()
    for code in range(-7, 1):
        assert L.sepconv_status_str(code)
    assert "sm_100a" in sc.version()
    assert sc.launch_count() == 0


@pytest.mark.parametrize("args,code", [
    ((16, 16, 0), "E_INVALID"),
    ((16, 16, 18), "E_UNSUPPORTED"),
    ((2, 16, 3), "E_INVALID"),
    ((16, 2, 3), "E_INVALID"),
])
def test_plan_validation_before_device(args, code):
    with pytest.raises(sc.SepconvError) as ei:
        sc.plan(*args)
    assert ei.value.code == code


def test_plan_ex_pitch_validation():
    with pytest.raises(sc.SepconvError) as ei:
        sc.plan_ex(1, 16, 16, 3, ld_in=8)
    assert ei.value.code == "E_INVALID"
    with pytest.raises(sc.SepconvError) as ei:
        sc.plan_ex(1, 16, 16, 3, ld_out=5)
    assert ei.value.code == "E_INVALID"
    with pytest.raises(sc.SepconvError) as ei:
        sc.plan_ex(0, 16, 16, 3)
    assert ei.value.code == "E_INVALID"


def test_plan_without_device_is_unsupported():
    torch = pytest.importorskip("torch")
    if torch.cuda.is_available():
        pytest.skip("has a GPU")
    with pytest.raises(sc.SepconvError) as ei:
        sc.plan(64, 64, 3)
    assert ei.value.code == "E_UNSUPPORTED"


@pytest.mark.parametrize("H,K,G", [(64, 3, 1), (64, 3, 2), (100, 5, 3), (16384, 17, 8), (16384, 3, 4), (1001, 9, 7)])
def test_band_matches_oracle_partition(H, K, G):
    ho = H - K + 1
    total_out, owned_sum = 0, 0
    for g in range(G):
        r0, rows, owned, alloc = sc.band(H, K, G, g)
        o0, o1 = oracle.band_rows(ho, G, g)
        assert (r0, rows) == (o0, o1 - o0)
        assert alloc == rows + K - 1
        assert owned == (rows + K - 1 if g == G - 1 else rows)
        total_out += rows
        owned_sum += owned
    assert total_out == ho
    assert owned_sum == H          # every input row owned by exactly one rank


def test_band_rejects_thin_bands():
    with pytest.raises(sc.SepconvError):
        sc.band(40, 17, 8, 0)       # 24 output rows / 8 = 3 < K-1 = 16
    with pytest.raises(sc.SepconvError):
        sc.band(40, 3, 2, 2)
    with pytest.raises(sc.SepconvError):
        sc.band(40, 18, 1, 0)


def test_band_single_gpu_is_whole_image():
    assert sc.band(100, 7, 1, 0) == (0, 94, 100, 100)


@pytest.mark.parametrize("n,G,halo", [(16384, 8, 8), (2048, 2, 6), (101, 3, 4), (1000, 7, 2), (64, 1, 8)])
def test_sor_band_partition(n, G, halo):
    covered = 0
    for g in range(G):
        r0, rows, a0, arows = sor.band(n, G, g, halo)
        assert r0 % 2 == 0 and a0 % 2 == 0                # colouring is band-invariant
        assert r0 == covered
        covered += rows
        assert a0 == (r0 - halo if g > 0 else r0)
        assert a0 + arows == (r0 + rows + halo if g < G - 1 else n)
        assert rows >= (halo if G > 1 else 1)
    assert covered == n


def test_sor_band_rejects_thin_bands_and_odd_halos():
    with pytest.raises(sc.SepconvError):
        sor.band(40, 8, 0, 8)
    with pytest.raises(sc.SepconvError):
        sor.band(400, 2, 0, 3)


# ---- the size selector's SELECT, pure host arithmetic --------------------------
def _sel(cutoffs, n_algos):
    algos = tuple(sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, i % 4) for i in range(n_algos))
    return sc.Selector(7, tuple(cutoffs), algos)


def test_select_follows_the_cutoff_definition():
    """SELECT(input, s) = alpha_i s.t. c_i > size >= c_{i-1}, c_0 = 0, c_m = inf:
    a size equal to a cutoff belongs to the level above it."""
    s = _sel([1000, 50000], 3)
    cases = {0: 0, 1: 0, 999: 0, 1000: 1, 1001: 1, 49999: 1, 50000: 2, 10 ** 12: 2}
    for size, level in cases.items():
        got = s.select(size)
        assert got.config == level % 4, (size, got)
        assert got.source == sc.SRC_SELECTOR
    one = _sel([], 1)
    assert one.select(0).config == 0 and one.select(2 ** 40).config == 0
    full = _sel([4 ** i for i in range(1, 12)], 12)           # 12 levels: the paper's maximum
    assert full.select(4 ** 11).config == 11 % 4 and full.select(4 ** 11 - 1).config == 10 % 4


@pytest.mark.parametrize("cutoffs,m", [([500, 500], 3), ([900, 100], 3), ([0], 2), ([], 0)])
def test_select_rejects_malformed_selectors(cutoffs, m):
    s = sc._Selector()
    s.k, s.m = 5, m
    for i, c in enumerate(cutoffs):
        s.cutoffs[i] = c
    out = sc._Choice()
    import ctypes
    assert sc.lib().sepconv_select(ctypes.byref(s), 100, ctypes.byref(out)) == -1   # E_INVALID


def test_choice_names_and_steal_field():
    """The Python Choice mirrors sepconv_choice_t field for field (sched_steal included) and names
    a schedule override as @p<parts>g<grid>[st<threshold>]."""
    c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 4, sched_parts=18, sched_grid=148, sched_steal=4)
    assert c.name == "sep-fused-tma4@p18g148st4"
    assert sc.Choice._from(c._c()) == c
    assert sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 2, sched_steal=4).name == "sep-fused-tma2"
    assert [f[0] for f in sc._Choice._fields_][-2:] == ["sched_steal", "source"]


def test_set_choice_validation_before_device():
    """sepconv_set_choice rejects a NULL plan, a NULL choice and a malformed one without a device."""
    import ctypes
    L = sc.lib()
    c = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 0)._c()
    assert L.sepconv_set_choice(None, 2, ctypes.byref(c)) == -1
    bad = sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, 99)._c()
    assert L.sepconv_set_choice(None, 2, ctypes.byref(bad)) == -1
    assert L.sepconv_set_choice(None, 2, None) == -1
