"""Shared test helpers (golden fixture parsing)."""
import os

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def read_golden(name):
    """Parse a tests/golden/*.txt fixture: '[section]' headers followed by rows of numbers,
    or 'key value  # citation' lines.  '#' starts a comment."""
    path = os.path.join(ROOT, "tests", "golden", name)
    sections, kv, cur = {}, {}, None
    with open(path) as f:
        for line in f:
            line = line.split("#", 1)[0].strip()
            if not line:
                continue
            if line.startswith("[") and line.endswith("]"):
                cur = line[1:-1]
                sections[cur] = []
                continue
            parts = line.split()
            if cur is not None:
                sections[cur].append([float(p) for p in parts])
            else:
                kv[parts[0]] = float(parts[1])
    return sections, kv
