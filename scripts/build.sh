# build libh2tap.so in-tree without importing the package (a stale .so would fail to load)
cd "$(dirname "$0")/.." && python -c "
import importlib.util
sp = importlib.util.spec_from_file_location('b', 'paper_conf_cidr_appuswamykpa17_b200/_build.py')
m = importlib.util.module_from_spec(sp); sp.loader.exec_module(m); m.build()"
