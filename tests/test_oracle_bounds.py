"""Pins for the bounds (oracle/bounds.py): closed forms and LP cross-checks."""
import pytest

from oracle import bounds

T_THR = {"POTRF": 3.0, "TRSM": 1.2, "SYRK": 1.1, "GEMM": 2.0}
T_LAT = {"POTRF": 5.0, "TRSM": 2.0, "SYRK": 1.5, "GEMM": 3.0}


@pytest.mark.parametrize("N", [1, 2, 4, 10, 20])
def test_mixed_dominates(N):
    for M in (1, 2, 8):
        a = bounds.area(N, T_THR, M)
        c = bounds.chain(N, T_LAT)
        m = bounds.mixed(N, T_THR, T_LAT, M)
        assert m >= a and m >= c and m == max(a, c)
        assert bounds.critical_path(N, T_LAT) >= c


@pytest.mark.parametrize("N", [2, 5, 12])
def test_lp_single_resource_equals_closed_form(N):
    T = {"gpu": T_THR}
    for M in (1, 3):
        lp = bounds.lp_area_mixed(N, T, {"gpu": M}, mixed_chain=False)
        assert abs(lp - bounds.area(N, T_THR, M)) < 1e-9 * lp
        lpm = bounds.lp_area_mixed(N, T, {"gpu": M}, mixed_chain=True)
        assert abs(lpm - max(bounds.area(N, T_THR, M), bounds.chain(N, T_THR))) < 1e-9 * lpm


def test_lp_related_platform_closed_form():
    """'Related' platform (L791-797): GPU exactly K times faster on every kernel ->
    area = W_cpu / (M_cpu + K M_gpu)."""
    N, K, Mc, Mg = 8, 7.0, 9, 3
    Tc = {"POTRF": 1.0, "TRSM": 3.0, "SYRK": 3.0, "GEMM": 6.0}
    Tg = {t: v / K for t, v in Tc.items()}
    W = bounds.area(N, Tc, 1)
    lp = bounds.lp_area_mixed(N, {"cpu": Tc, "gpu": Tg}, {"cpu": Mc, "gpu": Mg}, mixed_chain=False)
    assert abs(lp - W / (Mc + K * Mg)) < 1e-9 * lp


def test_critical_path_unit_weights():
    assert bounds.critical_path(7, {k: 1.0 for k in T_THR}) == 3 * 7 - 2


def test_gemm_peak():
    # R_G = 2 nb^3 / T_G; bound = (n^3/3) / (M R_G)
    n, nb = 9600, 960
    assert abs(bounds.gemm_peak(n, nb, 2.0, 1) - (n ** 3 / 3) / (2 * nb ** 3 / 2.0)) < 1e-9


def test_owner_area_pins():
    """Owner-area bound (SURVEY §8c ext): one rank = the area bound; the ranks' sums add up
    to the total work; with flop weights the max/mean imbalance is SURVEY §8e's table
    (2x4 / 4x2 / 1x8 at N = 48: 1.035 / 1.095 / 1.013; N = 96: 1.016 / 1.047 / 1.003)."""
    T = {"POTRF": 0.7, "TRSM": 1.9, "SYRK": 1.3, "GEMM": 2.6}
    for N in (1, 2, 5, 9):
        mx, w = bounds.owner_area(N, 1, 1, T)
        assert mx == pytest.approx(bounds.area(N, T, 1))
        for p, q in ((1, 2), (2, 2), (2, 3)):
            mx, w = bounds.owner_area(N, p, q, T)
            assert sum(w) == pytest.approx(bounds.area(N, T, 1))
            assert mx >= bounds.area(N, T, p * q) - 1e-12
    flops = {"POTRF": 1 / 3, "TRSM": 1.0, "SYRK": 1.0, "GEMM": 2.0}
    want = {(48, 2, 4): 1.035, (48, 4, 2): 1.095, (48, 1, 8): 1.013,
            (96, 2, 4): 1.016, (96, 4, 2): 1.047, (96, 1, 8): 1.003}
    for (N, p, q), v in want.items():
        mx, w = bounds.owner_area(N, p, q, flops)
        assert round(mx / (sum(w) / len(w)), 3) == v
