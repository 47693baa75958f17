"""Pins for the oracle's CHECKERS (oracle.rel_diff, oracle.backward_error) and for the
plain-Python replay oracle/sim.py itself -- each against values fixed by hand or by the
mathematics, never by the code under test.  Every float parity test of the GPU path rests
on rel_diff and backward_error, so a checker that returned 0, read the wrong triangle or
dropped a term must fail here.  CPU only."""
import math

import numpy as np
import pytest

import oracle
import spdgen
from oracle import dag, sim

EPS = np.finfo(np.float64).eps


# ----------------------------------------------------------------------------- rel_diff (reading R8)
REF = np.array([[2.0, 0.0, 0.0],
                [1.0, 3.0, 0.0],
                [1e-9, 4.0, 5.0]])


def test_rel_diff_identical_is_zero():
    d = oracle.rel_diff(REF.copy(), REF)
    assert d == {"max_rel_floored": 0.0, "max_rel": 0.0, "fro_rel": 0.0}


def test_rel_diff_hand_values_large_entry():
    """One lower entry off by 3e-10 relative: floored max = 3e-10 > the 1e-10 bar."""
    L = REF.copy()
    L[2, 1] = 4.0 * (1 + 3e-10)
    d = oracle.rel_diff(L, REF)
    assert d["max_rel_floored"] == pytest.approx(3e-10, rel=1e-6)
    assert d["max_rel_floored"] > 1e-10
    assert d["max_rel"] == pytest.approx(3e-10, rel=1e-6)
    assert d["fro_rel"] == pytest.approx(4.0 * 3e-10 / math.sqrt(4 + 1 + 9 + 1e-18 + 16 + 25), rel=1e-6)


def test_rel_diff_floor_on_tiny_entries():
    """A tiny reference entry (1e-9) is compared against the floor 1e-6 * max|ref| = 5e-6:
    an absolute error of 1e-9 gives 2e-4 floored (the unfloored ratio is 1)."""
    L = REF.copy()
    L[2, 0] = 2e-9
    d = oracle.rel_diff(L, REF)
    assert d["max_rel_floored"] == pytest.approx(1e-9 / 5e-6, rel=1e-9)
    assert d["max_rel"] == pytest.approx(1.0, rel=1e-9)


@pytest.mark.parametrize("pos", [(0, 0), (2, 2), (2, 0), (1, 0)])
def test_rel_diff_sees_every_lower_position(pos):
    """Corners and the diagonal: a 1e-8 relative change anywhere in the lower triangle of a
    bench-shaped factor is reported (a checker skipping rows / columns fails here)."""
    n = 97
    L0 = np.tril(spdgen.uniform_spd(n, 3))
    L0[np.diag_indices(n)] = np.abs(L0[np.diag_indices(n)])
    r, c = pos
    r, c = (n - 1 if r == 2 else r), (n - 1 if c == 2 else c)
    L = L0.copy()
    L[r, c] *= 1 + 1e-8
    assert oracle.rel_diff(L, L0)["max_rel_floored"] > 1e-10


def test_rel_diff_reads_the_lower_triangle_only():
    """The factor's strictly upper part is not part of L (reading R4): garbage there is not
    a difference, while a transposed factor (upper instead of lower) is a total mismatch."""
    L = REF.copy()
    L[0, 2] = 123.0
    assert oracle.rel_diff(L, REF)["max_rel_floored"] == 0.0
    d = oracle.rel_diff(REF.T.copy(), REF)
    assert d["max_rel_floored"] >= 1.0 and d["fro_rel"] > 0.5


# ----------------------------------------------------------------------------- backward_error
def test_backward_error_closed_form():
    """A = I, L = I + delta E_ij (i > j): L L^T - A = delta (E_ij + E_ji) + delta^2 E_ii, so
    ||A - L L^T||_F = sqrt(2 delta^2 + delta^4) and ||A||_F = sqrt(n)."""
    n, delta = 50, 1e-9
    A = np.eye(n)
    L = np.eye(n)
    L[7, 3] = delta
    want = math.sqrt(2 * delta ** 2 + delta ** 4) / (n * EPS * math.sqrt(n))
    assert oracle.backward_error(A, L) == pytest.approx(want, rel=1e-6)
    assert oracle.backward_error(A, L) > 10.0


def test_backward_error_exact_factor_is_zero():
    n = 120
    L0 = spdgen.integer_L0(n, 4)
    assert oracle.backward_error(spdgen.integer_spd(n, 4), L0) == 0.0


def test_backward_error_flags_a_perturbed_factor():
    """The north-star bar is 10; one diagonal entry of a uniform-family factor (~14) off by
    1e-10 relative moves A's (150, 150) entry by ~2 * 14 * 1.4e-9 = 4e-8 against
    n eps ||A||_F ~ 1.3e-10, far above the bar (the LAPACK factor itself is well below it)."""
    n = 200
    A = spdgen.uniform_spd(n, 9)
    L = np.linalg.cholesky(A)
    assert oracle.backward_error(A, L) <= 10.0
    Lp = L.copy()
    Lp[150, 150] *= 1 + 1e-10
    assert oracle.backward_error(A, Lp) > 10.0


def test_backward_error_uses_only_the_lower_triangle_of_A():
    n = 64
    A = spdgen.uniform_spd(n, 2)
    L = np.linalg.cholesky(A)
    An = spdgen.uniform_spd(n, 2, upper="nan")
    assert oracle.backward_error(An, L) == oracle.backward_error(A, L)
    assert oracle.backward_error(A, L.T.copy()) > 1e6  # L^T L != A


# ----------------------------------------------------------------------------- oracle/sim.py itself
TYPES = ("POTRF", "TRSM", "SYRK", "GEMM")


@pytest.mark.parametrize("policy", [0, 1])
@pytest.mark.parametrize("N", [1, 3, 6])
def test_sim_one_worker_is_the_serial_sum(policy, N):
    T = [3.0, 1.25, 1.5, 2.0]
    cnt = dag.counts(N)
    serial = cnt["POTRF"] * T[0] + cnt["TRSM"] * T[1] + cnt["SYRK"] * T[2] + cnt["GEMM"] * T[3]
    mk, out = sim.simulate(N, [1], [T], policy=policy)
    assert mk == serial
    assert len(out) == len(dag.tasks(N))


@pytest.mark.parametrize("policy", [0, 1])
def test_sim_unlimited_workers_unit_weights_is_3N_minus_2(policy):
    """with unit task times the longest chain has 3N-2 tasks."""
    for N in (1, 2, 5, 9):
        mk, _ = sim.simulate(N, [len(dag.tasks(N))], [[1, 1, 1, 1]], policy=policy)
        assert mk == 3 * N - 2


@pytest.mark.parametrize("policy", [0, 1])
def test_sim_unlimited_workers_flop_weights_is_3N_minus_10_thirds(policy):
    """Flop-proportional times (nb^3 units: POTRF 1/3, TRSM 1, SYRK 1, GEMM 2) -- the longest
    path is 3N - 10/3 (along the last tile row)."""
    for N in (3, 5, 8):
        mk, _ = sim.simulate(N, [len(dag.tasks(N))], [[1 / 3, 1.0, 1.0, 2.0]], policy=policy)
        assert mk == pytest.approx(3 * N - 10 / 3, abs=1e-12)


# N = 3 worked by hand: one "CPU" (class 0: P 4, T 3, S 3, G 6) and one
# "GPU" (class 1: P 2, T 2, S 1, G 1); workers numbered class by class (w0 CPU, w1 GPU).
HAND_TIMES = [[4.0, 3.0, 3.0, 6.0], [2.0, 2.0, 1.0, 1.0]]
# dmda: ready tasks assigned in release order to the minimum completion estimate.
#   t=0 P0 -> w1 (2 < 4).  t=2 T10 -> w1 (4 < 5), T20 -> w0 (5 < 6).  t=4 S10 -> w1 (5).
#   t=5 (T20 on w0 and S10 on w1 end together; w0's successors released first):
#       G210 -> w1 (6 < 11), S20 -> w1 (7 < 8), P1 -> w0 (tie 9 = 9: lowest worker).
#   t=9 T21 -> w1 (11 < 12).  t=11 S21 -> w1 (12).  t=12 P2 -> w1 (14 < 16).
HAND_DMDA = {("P", 0, 0, 0): (1, 0, 2), ("T", 1, 0, 0): (1, 2, 4), ("T", 2, 0, 0): (0, 2, 5),
             ("S", 1, 1, 0): (1, 4, 5), ("G", 2, 1, 0): (1, 5, 6), ("S", 2, 2, 0): (1, 6, 7),
             ("P", 1, 1, 1): (0, 5, 9), ("T", 2, 1, 1): (1, 9, 11), ("S", 2, 2, 1): (1, 11, 12),
             ("P", 2, 2, 2): (1, 12, 14)}
# dmdas: bottom levels with the fastest times (P2 2, S21 3, T21 5, P1 7, S20 4, G210 6, S10 8,
#   T20 8, T10 10, P0 12); ready tasks and worker queues in priority order.
#   t=5: P1 -> w1 (7 < 9), G210 -> w1 (8 < 11), S20 -> w0 (8 < 9); w1 runs P1 first.
#   t=7 G210 on w1.  t=8 T21 -> w1 (10 < 11).  t=10 S21 -> w1 (11).  t=11 P2 -> w1 (13).
HAND_DMDAS = {("P", 0, 0, 0): (1, 0, 2), ("T", 1, 0, 0): (1, 2, 4), ("T", 2, 0, 0): (0, 2, 5),
              ("S", 1, 1, 0): (1, 4, 5), ("G", 2, 1, 0): (1, 7, 8), ("S", 2, 2, 0): (0, 5, 8),
              ("P", 1, 1, 1): (1, 5, 7), ("T", 2, 1, 1): (1, 8, 10), ("S", 2, 2, 1): (1, 10, 11),
              ("P", 2, 2, 2): (1, 11, 13)}


@pytest.mark.parametrize("policy,want,mk_want", [(0, HAND_DMDA, 14.0), (1, HAND_DMDAS, 13.0)])
def test_sim_hand_worked_two_class_schedule(policy, want, mk_want):
    mk, out = sim.simulate(3, [1, 1], HAND_TIMES, policy=policy)
    assert mk == mk_want
    ts = dag.tasks(3)
    letter = "PTSG"
    got = {}
    for idx, (w, cls, t0, t1) in out.items():
        t = ts[idx]
        key = (letter[t.type], t.i, t.j, t.k)
        got[key] = (w, t0, t1)
        assert cls == w  # one worker per class
    assert got == want
