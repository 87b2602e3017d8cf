"""Pins for the mat-vec oracle."""
import os

import numpy as np

import gen
import oracle


def test_integer_valued_exact(shmdir):
    m = gen.matrix_files(shmdir, 37, 4099, seed=3, integer=True)
    A = np.fromfile(m["A"], dtype="<f4").reshape(37, 4099).astype(np.int64)
    x = np.fromfile(m["x"], dtype="<f4").astype(np.int64)
    y = oracle.matvec(m["A"], m["x"], 37, 4099, nthreads=3)
    assert np.array_equal(y, (A @ x).astype(np.float64))  # integer closed form


def test_closed_form_ones(shmdir):
    a = os.path.join(shmdir, "A.f32"); x = os.path.join(shmdir, "x.f32")
    np.ones((5, 1000), "<f4").tofile(a)
    np.full(1000, 0.5, "<f4").tofile(x)
    assert oracle.matvec(a, x, 5, 1000).tolist() == [500.0] * 5


def test_random_against_float64_library(shmdir):
    m = gen.matrix_files(shmdir, 64, 131072 // 8, seed=3)
    A = np.fromfile(m["A"], dtype="<f4").reshape(64, -1).astype(np.float64)
    x = np.fromfile(m["x"], dtype="<f4").astype(np.float64)
    y = oracle.matvec(m["A"], m["x"], 64, A.shape[1], row0=10, nrows=20)
    ref = A[10:30] @ x
    assert np.max(np.abs(y - ref) / np.abs(ref)) < 1e-12
