"""Pins for the task graph (oracle/dag.py) against what the paper prints."""
import math
import os

import pytest

from oracle import bounds, dag

GOLD = os.path.join(os.path.dirname(__file__), "golden")


def _golden(name):
    with open(os.path.join(GOLD, name)) as f:
        return [ln.split() for ln in f if ln.strip() and not ln.startswith("#")]


def test_fig1_task_names_exact():
    """Fig. 1: the 35 tasks of the 5x5 tiled matrix."""
    gold = {r[0] for r in _golden("fig1_tasks_5x5.txt")}
    assert len(gold) == 35
    assert {t.name for t in dag.tasks(5)} == gold


def test_acceleration_factor_K():
    """K values printed on L817-819 reproduce from the task counts + Table I."""
    for N, K in _golden("k_values.txt"):
        assert f"{dag.acceleration_factor_K(int(N)):.2f}" == K


@pytest.mark.parametrize("N", list(range(1, 13)))
def test_counts_closed_form(N):
    c = dag.counts(N)
    assert c == bounds.task_counts(N)
    assert c["POTRF"] == N and c["TRSM"] == c["SYRK"] == N * (N - 1) // 2
    assert c["GEMM"] == math.comb(N, 3)


@pytest.mark.parametrize("N", [1, 2, 3, 5, 10, 20])
def test_edge_count_and_in_degrees(N):
    ts, E = dag.edges(N)
    NG = math.comb(N, 3)
    expect = (N - 1) + 2 * (N * (N - 1) // 2 + (N - 1) * (N - 2) // 2) + 2 * NG + math.comb(N - 1, 3)
    assert len(E) == expect
    deg = dag.in_degrees(N)
    for t, d in zip(ts, deg):
        first = t.k == 0
        want = {dag.POTRF: 0 if first else 1, dag.TRSM: 1 if first else 2,
                dag.SYRK: 1 if first else 2, dag.GEMM: 2 if first else 3}[t.type]
        assert d == want, (t.name, d)


def test_edge_counts_known_values():
    assert len(dag.edges(5)[1]) == 60
    assert len(dag.edges(20)[1]) == 3990


@pytest.mark.parametrize("N", [1, 2, 3, 4, 8, 12])
def test_unit_weight_longest_path_is_diagonal_chain(N):
    """L383-386: the path with all N POTRFs, N-1 TRSMs and N-1 SYRKs; with unit
    weights it is a longest path: 3N - 2 tasks."""
    assert dag.longest_path(N, lambda t: 1.0) == 3 * N - 2


@pytest.mark.parametrize("N", [3, 4, 8, 12])
def test_flop_weight_longest_path(N):
    """With flop weights (nb^3 units: 1/3, 1, 1, 2) the longest path runs along the
    last tile row: 3N - 10/3 (reading R12), longer than the chain N/3 + 2(N-1)."""
    w = [1 / 3, 1.0, 1.0, 2.0]
    lp = dag.longest_path(N, lambda t: w[t.type])
    assert abs(lp - (3 * N - 10 / 3)) < 1e-12
    assert lp >= N / 3 + 2 * (N - 1) - 1e-12


def test_successor_counts():
    """POTRF_k -> N-k-1 successors, TRSM_i_k -> N-k-1, SYRK / GEMM -> exactly 1
    (except the final POTRF, an exit)."""
    N = 10
    ts, E = dag.edges(N)
    out = [0] * len(ts)
    for p, _ in E:
        out[p] += 1
    for t, o in zip(ts, out):
        if t.type in (dag.POTRF, dag.TRSM):
            assert o == N - t.k - 1, t.name
        else:
            assert o == 1, t.name


def test_bottom_level_exit_and_monotone():
    N = 6
    ts, E = dag.edges(N)
    bl = dag.bottom_levels(N, lambda t: 1.0)
    assert bl[-1] == 1.0  # POTRF_{N-1} is the only exit
    for p, s in E:
        assert bl[p] >= bl[s] + 1.0
    assert max(bl) == 3 * N - 2
