#!/usr/bin/env python
"""Build A/B variants of libh2tap.so with extra preprocessor defines into variants/ (git-ignored
.so files; they travel to the GPU box with the gpurun snapshot). Run one with H2TAP_LIB=<path>.
usage: python scripts/build_variants.py name=DEF1,DEF2 [name2=...]
e.g.   python scripts/build_variants.py hr_lazy=HR_EAGER=0 hr_u2=HR_U=2"""
import os
import sys
from concurrent.futures import ThreadPoolExecutor

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cidr_appuswamykpa17_b200 import _build  # noqa: E402


def one(spec):
    name, _, defs = spec.partition("=")
    out = os.path.join(ROOT, "variants", f"libh2tap_{name}.so")
    os.makedirs(os.path.dirname(out), exist_ok=True)
    _build.build(force=True, defines=[d for d in defs.split(",") if d], out=out)
    return out


if __name__ == "__main__":
    with ThreadPoolExecutor(2) as ex:
        for p in ex.map(one, sys.argv[1:]):
            print(p)
