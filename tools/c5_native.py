"""Build and run tools/c5_native.cpp (config C5 with a native C++ OLTP driver, epoch cutter and
query loop; see its header). Usage: python tools/c5_native.py [--out F] -- [c5_native args]"""
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SRC = os.path.join(ROOT, "tools", "c5_native.cpp")
EXE = os.path.join(ROOT, "build", "c5_native")
PKG = os.path.join(ROOT, "paper_conf_cidr_appuswamykpa17_b200")


def build() -> str:
    lib = os.path.join(PKG, "libh2tap.so")
    if not os.path.exists(lib):
        raise RuntimeError("libh2tap.so missing: run __graft_entry__.build() first")
    if os.path.exists(EXE) and os.path.getmtime(EXE) >= max(os.path.getmtime(SRC), os.path.getmtime(lib)):
        return EXE
    os.makedirs(os.path.dirname(EXE), exist_ok=True)
    subprocess.check_call(["g++", "-O2", "-std=c++17", "-pthread", "-Wall", "-I", os.path.join(ROOT, "include"),
                           SRC, "-o", EXE, "-L", PKG, "-l:libh2tap.so", f"-Wl,-rpath,{PKG}"])
    return EXE


def main():
    argv = sys.argv[1:]
    out = None
    if "--out" in argv:
        i = argv.index("--out")
        out = argv[i + 1]
        del argv[i:i + 2]
    if argv and argv[0] == "--":
        argv = argv[1:]
    r = subprocess.run([build()] + argv, capture_output=True, text=True)
    sys.stderr.write(r.stderr)
    line = r.stdout.strip().splitlines()[-1] if r.stdout.strip() else ""
    print(line)
    if out and line:
        with open(out, "w") as f:
            f.write(line + "\n")
    return r.returncode


if __name__ == "__main__":
    sys.exit(main())
