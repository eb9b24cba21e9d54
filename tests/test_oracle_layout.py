"""Pins of the NEXT-3 layout oracle (§5.3: SUM(col1 + ... + colN) over DSM / PAX / NSM),
none using the oracle's own address arithmetic: numpy's sum over the logical matrix (the layouts are
built by numpy reshapes/transposes in chgen), a closed form, and pure-Python loops on tiny tables."""
import numpy as np
import pytest

import chgen
import oracle

LAYOUTS = ("dsm", "pax", "nsm")


@pytest.mark.parametrize("n", [0, 1, 3, 64, 65, 1000, 4099])
@pytest.mark.parametrize("cols", [[0], [0, 1], [0, 1, 2, 3], list(range(8)), list(range(16)), [15], [3, 7, 12]])
def test_matches_numpy_on_every_layout(n, cols):
    m = chgen.layout_matrix(n, 16, seed=n + 1)
    want = int(m[:, cols].astype(np.int64).sum()) if n else None
    for lay in LAYOUTS:
        data = chgen.encode_layout(m, lay)
        assert oracle.layout_sum(data, lay, n, 16, cols) == want, lay
    if n:  # DSM with padded column starts, PAX with 16-row minipages
        assert oracle.layout_sum(chgen.encode_layout(m, "dsm", col_stride=n + 13), "dsm", n, 16, cols,
                                 col_stride=n + 13) == want
        assert oracle.layout_sum(chgen.encode_layout(m, "pax", pax_rows=16), "pax", n, 16, cols,
                                 pax_rows=16) == want


def test_closed_form():
    """value(r, c) = r * ncols + c  =>  SUM over S = |S| * ncols * n(n-1)/2 + n * sum(S)."""
    n, k = 5000, 16
    m = (np.arange(n, dtype=np.int64)[:, None] * k + np.arange(k)[None, :]).astype(np.int32)
    for cols in ([0], [1, 2], list(range(16)), [5, 9, 15]):
        want = len(cols) * k * n * (n - 1) // 2 + n * sum(cols)
        for lay in LAYOUTS:
            assert oracle.layout_sum(chgen.encode_layout(m, lay), lay, n, k, cols) == want


def test_brute_force_tiny():
    """Python loops over records, reading each attribute where the paper places it (L968-972)."""
    n, k, mp = 37, 8, 4
    m = chgen.layout_matrix(n, k, seed=9)
    cols = [1, 4, 6]
    nsm, dsm, pax = (chgen.encode_layout(m, x, pax_rows=mp) for x in ("nsm", "dsm", "pax"))
    for r in range(n):  # the encodings place record r, attribute c where the paper says
        for c in range(k):
            assert nsm[r * k + c] == dsm[c * n + r] == pax[(r // mp) * k * mp + c * mp + r % mp] == m[r, c]
    want = sum(int(m[r, c]) for r in range(n) for c in cols)
    assert oracle.layout_sum(pax, "pax", n, k, cols, pax_rows=mp) == want
    assert oracle.layout_sum(nsm, "nsm", n, k, cols) == want


def test_paper_page_geometry():
    """PAX page = 16 minipages x 64 values x 4 B = 4 KB (L970-972)."""
    m = chgen.layout_matrix(128, 16, seed=2)
    assert chgen.encode_layout(m, "pax").nbytes == 2 * 4096
