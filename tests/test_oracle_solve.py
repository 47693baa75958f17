"""Pins for the oracle's solve (A = L L^T used to solve A X = B,
PAPER.md L166-171): LAPACK dpotrs (scipy cho_solve), exact integer solutions, the
residual bound, and the 1 x 1 closed form."""
import numpy as np
import pytest
import scipy.linalg as sla

import oracle
import spdgen


@pytest.mark.parametrize("n,nrhs", [(1, 1), (7, 3), (64, 1), (300, 40), (512, 5)])
def test_solve_matches_lapack(n, nrhs):
    A = spdgen.uniform_spd(n, 4)
    L = np.linalg.cholesky(A)
    B = spdgen.rhs(n, nrhs, 2)
    X = oracle.chol_solve(L, B)
    ref = sla.cho_solve((L, True), B)
    assert np.max(np.abs(X - ref)) <= 1e-13 * max(1.0, np.max(np.abs(ref)))


@pytest.mark.parametrize("n,seed", [(40, 0), (257, 3), (960, 1)])
def test_integer_solution_exact(n, seed):
    """A = L0 L0^T and B = A X0 are exact integers; substitution with L0 (diagonal in
    {1, 2, 4}) returns X0 bit for bit."""
    L0 = spdgen.integer_L0(n, seed)
    A = spdgen.integer_spd(n, seed)
    X0 = spdgen.integer_rhs_solution(n, 6, seed)
    B = A @ X0
    assert np.array_equal(B, np.round(B))
    assert np.array_equal(oracle.chol_solve(L0, B), X0)


def test_residual_and_closed_form():
    n, nrhs = 400, 7
    A = spdgen.uniform_spd(n, 9)
    L, info = oracle.chol_tiled(A, 100)
    assert info == 0
    B = spdgen.rhs(n, nrhs, 1)
    X = oracle.chol_solve(L, B)
    eps = np.finfo(np.float64).eps
    r = np.linalg.norm(A @ X - B) / (np.linalg.norm(A) * np.linalg.norm(X) * n * eps)
    assert r <= 10.0
    # 1 x 1: x = b / l^2
    assert oracle.chol_solve(np.array([[2.0]]), np.array([[6.0]]))[0, 0] == 1.5
    # a transposed factor (a plausible mistake) is caught by the LAPACK pin
    Xbad = oracle.chol_solve(np.ascontiguousarray(L.T), B)
    assert np.max(np.abs(Xbad - X)) > 1e-6
