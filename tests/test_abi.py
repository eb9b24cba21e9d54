"""CPU checks of the C-ABI library: it loads, exports every symbol include/h2tap.h declares,
and rejects bad calls without a GPU (no compute calls here)."""
import os
import re

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def h():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


def header_functions():
    src = open(os.path.join(ROOT, "include", "h2tap.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(h2tap_[a-z0-9_]+)\s*\(", src)))


def test_exports_every_declared_symbol(h):
    declared = header_functions()
    assert "h2tap_load_snapshot" in declared and "h2tap_run_query" in declared and "h2tap_free" in declared
    missing = [s for s in declared if not hasattr(h._lib, s)]
    assert not missing, missing
    assert sorted(h.ABI_SYMBOLS) == declared


def test_struct_layouts_match_header(h, tmp_path):
    """ctypes mirrors of the ABI structs have the C compiler's sizes and offsets."""
    import ctypes as C
    import subprocess
    structs = {"h2tap_column": h.h2tap_column, "h2tap_table": h.h2tap_table,
               "h2tap_config": h.h2tap_config, "h2tap_result": h.h2tap_result,
               "h2tap_field": h.h2tap_field, "h2tap_row_table": h.h2tap_row_table,
               "h2tap_query": h.h2tap_query, "h2tap_update": h.h2tap_update,
               "h2tap_store_stats": h.h2tap_store_stats, "h2tap_layout_table": h.h2tap_layout_table}
    lines = ['#include <stdio.h>', '#include <stddef.h>', '#include "h2tap.h"', 'int main(void){']
    for name, cls in structs.items():
        lines.append(f'printf("{name} %zu\\n", sizeof({name}));')
        for fname, _ in cls._fields_:
            lines.append(f'printf("{name}.{fname} %zu\\n", offsetof({name}, {fname}));')
    lines.append("return 0;}")
    src = tmp_path / "layout.c"
    src.write_text("\n".join(lines))
    exe = tmp_path / "layout"
    subprocess.check_call(["gcc", "-I", os.path.join(ROOT, "include"), str(src), "-o", str(exe)])
    got = dict(l.rsplit(" ", 1) for l in subprocess.check_output([str(exe)], text=True).split("\n") if l)
    for name, cls in structs.items():
        assert int(got[name]) == C.sizeof(cls), name
        for fname, _ in cls._fields_:
            assert int(got[f"{name}.{fname}"]) == getattr(cls, fname).offset, (name, fname)


def test_c_last_syllables(h):
    syl = ["BAR", "OUGHT", "ABLE", "PRI", "PRES", "ESE", "ANTI", "CALLY", "ATION", "EING"]
    for code in (0, 1, 99, 371, 500, 999):
        assert h.h2tap_c_last_name(code) == syl[code // 100] + syl[code // 10 % 10] + syl[code % 10]
    names = {h.h2tap_c_last_name(c) for c in range(1000)}
    assert len(names) == 1000  # injective: codes compare like strings for equality (R21)
    with pytest.raises(ValueError):
        h.h2tap_c_last_name(1000)


def test_bad_calls_fail_cleanly_without_gpu(h):
    import torch
    if torch.cuda.is_available():
        pytest.skip("CPU-only check")
    with pytest.raises(h.H2tapError) as ei:
        h.h2tap_open(0)
    assert ei.value.status == h.H2TAP_ECUDA
    assert "CUDA" in h.h2tap_last_error() or "cuda" in h.h2tap_last_error()
    import ctypes as C
    assert h._lib.h2tap_run_query(None, 6, None, 0, None) == h.H2TAP_EINVAL
    assert h._lib.h2tap_load_snapshot(None, None, 0, 1) == h.H2TAP_EINVAL
    assert h._lib.h2tap_open(None, None) == h.H2TAP_EINVAL
    assert h._lib.h2tap_refresh(None, None, 0, None, 0, 1, 0) == h.H2TAP_EINVAL
    assert h._lib.h2tap_refresh_rows(None, None, 0, None, 0, 1, 0) == h.H2TAP_EINVAL
    assert h._lib.h2tap_get_store_stats(None, None) == h.H2TAP_EINVAL
    h._lib.h2tap_free(None)
    h._lib.h2tap_close(None)


def test_no_oracle_in_product_path():
    """The product package must not import, link or read anything under oracle/."""
    pkg = os.path.join(ROOT, "paper_conf_cidr_appuswamykpa17_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h")):
                txt = open(os.path.join(dirpath, f)).read()
                assert "import oracle" not in txt and "from oracle" not in txt, f
                assert "oracle.h" not in txt and "liboracle" not in txt, f


def test_sass_is_sm100a_with_tma_bulk_copies(h):
    """The library is built for sm_100a only, and the scan kernels stream columns with TMA bulk
    copies (SASS UBLKCP from cp.async.bulk; B200_PROFILING.md 'What proves a Blackwell-native
    kernel')."""
    import shutil
    import subprocess
    cuobjdump = shutil.which("cuobjdump") or "/usr/local/cuda/bin/cuobjdump"
    if not os.path.exists(cuobjdump):
        pytest.skip("cuobjdump not available")
    sass = subprocess.run([cuobjdump, "-sass", h.LIB_PATH], capture_output=True, text=True).stdout
    archs = set(re.findall(r"arch = (sm_\w+)", sass))
    assert archs == {"sm_100a"}, archs
    assert "UBLKCP" in sass
    funcs = re.findall(r"Function : (\S+)", sass)
    assert any("q6_tma_kernel" in f for f in funcs) and any("q1_tma_kernel" in f for f in funcs)
